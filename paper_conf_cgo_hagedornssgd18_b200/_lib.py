"""ctypes binding of include/stencil.h — argument marshalling only.

Function names are the C-ABI names.  Every step of the stencil runs inside
libstencil.so's CUDA kernels; there is no Python or CPU fallback: importing
this module fails loudly when the library has not been built
(``python -m paper_conf_cgo_hagedornssgd18_b200.build``).
"""
from __future__ import annotations

import ctypes as C
import os
from typing import Optional, Sequence

import numpy as np

_PKG = os.path.dirname(os.path.abspath(__file__))
# LIFT_LIB_TAG=x loads the in-tree A/B build libstencil_x.so (build.py with
# the same variable); the default is the product library
_TAG = os.environ.get("LIFT_LIB_TAG", "")
LIB_PATH = os.path.join(_PKG, f"libstencil_{_TAG}.so" if _TAG else "libstencil.so")

if not os.path.exists(LIB_PATH):
    raise ImportError(f"{LIB_PATH} is missing: build it with `python __graft_entry__.py` or "
                      "`python paper_conf_cgo_hagedornssgd18_b200/build.py` (no CPU fallback exists)")
_lib = C.CDLL(LIB_PATH)

# status / enums (include/stencil.h)
STENCIL_OK, STENCIL_E_INVALID, STENCIL_E_UNSUPPORTED, STENCIL_E_CUDA, STENCIL_E_NOMEM = range(5)
PAD_CLAMP, PAD_MIRROR, PAD_WRAP, PAD_CONSTANT, PAD_REFLECT, PAD_DAMPEN = range(6)
OP_WEIGHTED, OP_HOTSPOT3D, OP_SRAD1, OP_SRAD2, OP_ACOUSTIC, OP_HOTSPOT2D, OP_GRADIENT, OP_SRAD = range(8)
(VARIANT_AUTO, VARIANT_GENERIC, VARIANT_TILE2D, VARIANT_SWEEP3D, VARIANT_PERSIST3D, VARIANT_GATHER,
 VARIANT_RESIDENT3D) = -1, 0, 1, 2, 3, 4, 5
OP_ARITY = {OP_WEIGHTED: 1, OP_HOTSPOT3D: 2, OP_SRAD1: 1, OP_SRAD2: 2, OP_ACOUSTIC: 2, OP_HOTSPOT2D: 2, OP_GRADIENT: 1, OP_SRAD: 1}

_P = C.c_void_p
_I64P = C.POINTER(C.c_int64)
_I32P = C.POINTER(C.c_int32)
_FP = C.POINTER(C.c_float)
_FPP = C.POINTER(C.c_void_p)


def _sig(name, res, args):
    f = getattr(_lib, name)
    f.restype = res
    f.argtypes = args
    return f


_create = _sig("stencil_plan_create", C.c_int, [C.POINTER(_P), C.c_int, C.c_int, _I64P, _I32P, _I32P, _I32P,
                                                 _I32P, _I32P, C.c_float, C.c_int32, _FP, _FP, C.c_int32])
_out_ext = _sig("stencil_plan_output_extents", C.c_int, [_P, _I64P])
_set_slab = _sig("stencil_plan_set_slab", C.c_int, [_P, C.c_int64, C.c_int64, C.c_int32])
_set_variant = _sig("stencil_plan_set_variant", C.c_int, [_P, C.c_int32])
_variant = _sig("stencil_plan_variant", C.c_int32, [_P])
_last_variant = _sig("stencil_plan_last_variant", C.c_int32, [_P])
_set_decay = _sig("stencil_plan_set_pad_decay", C.c_int, [_P, C.c_float])
_set_tb = _sig("stencil_plan_set_time_block", C.c_int, [_P, C.c_int32])
_tb = _sig("stencil_plan_time_block", C.c_int32, [_P])
_apply = _sig("stencil_apply", C.c_int, [_P, _FPP, C.c_int32, _P, _P])
_apply_region = _sig("stencil_apply_region", C.c_int, [_P, _FPP, C.c_int32, _P, C.c_int64, C.c_int64, _P])
_apply2_region = _sig("stencil_apply2_region", C.c_int, [_P, _P, _P, C.c_int64, C.c_int64, _P])
_apply_region_put = _sig("stencil_apply_region_put", C.c_int, [_P, _FPP, C.c_int32, _P, C.c_int64, C.c_int64, _P, _P,
                                                              _P, _P, C.c_uint32, _P])
_slab_step_fused = _sig("stencil_slab_step_fused", C.c_int, [_P, _FPP, C.c_int32, _P, _P, _P, _P, _P, C.c_uint32,
                                                            _P, _P, C.c_uint32, _P])
_wait_signals = _sig("stencil_wait_signals", C.c_int, [_P, _P, C.c_uint32, _P])
_iterate = _sig("stencil_iterate", C.c_int, [_P, _FPP, C.c_int32, _FPP, C.c_int32, C.c_int32, _P, _I32P])
_set_wait_timeout = _sig("stencil_set_wait_timeout_ms", C.c_int, [C.c_uint32])
_device_fault = _sig("stencil_device_fault", C.c_int, [])
_run_host = _sig("stencil_run_host", C.c_int, [_P, _FPP, C.c_int32, _FPP, C.c_int32, C.c_int32, _P, _P])
_run_host_batch = _sig("stencil_run_host_batch", C.c_int, [_P, _FPP, C.c_int32, _FPP, C.c_int32, C.c_int32,
                                                         C.c_int32, _FPP])
_destroy = _sig("stencil_plan_destroy", None, [_P])
_last_kernel = _sig("stencil_plan_last_kernel", C.c_char_p, [_P])
_status_string = _sig("stencil_status_string", C.c_char_p, [C.c_int])
_last_error = _sig("stencil_last_error", C.c_char_p, [])
_version = _sig("stencil_version", C.c_char_p, [])

EXPORTED = ("stencil_plan_create", "stencil_plan_output_extents", "stencil_plan_set_slab",
            "stencil_plan_set_variant", "stencil_plan_variant", "stencil_plan_last_variant",
            "stencil_plan_set_pad_decay", "stencil_plan_last_kernel",
            "stencil_plan_set_time_block",
            "stencil_plan_time_block", "stencil_apply", "stencil_apply_region", "stencil_apply2_region",
            "stencil_apply_region_put", "stencil_slab_step_fused", "stencil_wait_signals",
            "stencil_set_wait_timeout_ms", "stencil_device_fault",
            "stencil_iterate", "stencil_run_host", "stencil_run_host_batch", "stencil_plan_destroy",
            "stencil_status_string",
            "stencil_last_error", "stencil_version")


class StencilError(RuntimeError):
    def __init__(self, status: int, where: str):
        self.status = status
        msg = _status_string(status).decode()
        detail = _last_error().decode()
        super().__init__(f"{where}: {msg}: {detail}")


def _check(status: int, where: str):
    if status != STENCIL_OK:
        raise StencilError(status, where)


def _arr(ctype, vals):
    vals = list(vals)
    return (ctype * max(1, len(vals)))(*vals)


def _ptrs(ps: Sequence[int]):
    return (C.c_void_p * max(1, len(ps)))(*[C.c_void_p(int(p)) for p in ps])


def stencil_version() -> str:
    return _version().decode()


def stencil_status_string(status: int) -> str:
    return _status_string(status).decode()


def stencil_last_error() -> str:
    return _last_error().decode()


def stencil_plan_create(device: int, extents, size, step, pad_lo, pad_hi, kind, pad_value: float, op: int,
                        weights: Optional[np.ndarray] = None, params: Sequence[float] = ()) -> int:
    nd = len(extents)
    h = _P()
    w = None
    if weights is not None:
        w = np.ascontiguousarray(np.asarray(weights, np.float32).reshape(-1))
    prm = np.ascontiguousarray(np.asarray(list(params), np.float32))
    st = _create(C.byref(h), int(device), nd, _arr(C.c_int64, extents), _arr(C.c_int32, size),
                 _arr(C.c_int32, step), _arr(C.c_int32, pad_lo), _arr(C.c_int32, pad_hi),
                 _arr(C.c_int32, kind), float(pad_value), int(op),
                 None if w is None else w.ctypes.data_as(_FP),
                 prm.ctypes.data_as(_FP) if prm.size else None, int(prm.size))
    _check(st, "stencil_plan_create")
    return h.value


def stencil_plan_output_extents(plan: int, ndim: int):
    out = (C.c_int64 * 3)()
    _check(_out_ext(plan, out), "stencil_plan_output_extents")
    return tuple(int(out[i]) for i in range(ndim))


def stencil_plan_set_slab(plan: int, z_offset: int, global_n0: int, ghost: int):
    _check(_set_slab(plan, int(z_offset), int(global_n0), int(ghost)), "stencil_plan_set_slab")


def stencil_plan_set_variant(plan: int, variant: int):
    _check(_set_variant(plan, int(variant)), "stencil_plan_set_variant")


def stencil_plan_variant(plan: int) -> int:
    return int(_variant(plan))


def stencil_plan_set_pad_decay(plan: int, decay: float):
    _check(_set_decay(plan, float(decay)), "stencil_plan_set_pad_decay")


def stencil_plan_last_variant(plan: int) -> int:
    return int(_last_variant(plan))


def stencil_plan_set_time_block(plan: int, steps: int):
    _check(_set_tb(plan, int(steps)), "stencil_plan_set_time_block")


def stencil_plan_time_block(plan: int) -> int:
    return int(_tb(plan))


def stencil_apply(plan: int, inputs: Sequence[int], out: int, stream: int = 0):
    _check(_apply(plan, _ptrs(inputs), len(inputs), C.c_void_p(int(out)), C.c_void_p(int(stream))),
           "stencil_apply")


def stencil_apply_region(plan: int, inputs: Sequence[int], out: int, o0_begin: int, o0_end: int,
                         stream: int = 0):
    _check(_apply_region(plan, _ptrs(inputs), len(inputs), C.c_void_p(int(out)), int(o0_begin), int(o0_end),
                         C.c_void_p(int(stream))), "stencil_apply_region")


def stencil_apply2_region(plan: int, inp: int, out: int, o0_begin: int, o0_end: int, stream: int = 0):
    _check(_apply2_region(plan, C.c_void_p(int(inp)), C.c_void_p(int(out)), int(o0_begin), int(o0_end),
                          C.c_void_p(int(stream))), "stencil_apply2_region")


def stencil_apply_region_put(plan: int, inputs: Sequence[int], out: int, o0_begin: int, o0_end: int,
                             put_lo: int = 0, put_hi: int = 0, sig_lo: int = 0, sig_hi: int = 0, sig_value: int = 0,
                             stream: int = 0):
    v = lambda x: C.c_void_p(int(x)) if x else None
    _check(_apply_region_put(plan, _ptrs(inputs), len(inputs), C.c_void_p(int(out)), int(o0_begin), int(o0_end),
                             v(put_lo), v(put_hi), v(sig_lo), v(sig_hi), int(sig_value) & 0xffffffff,
                             C.c_void_p(int(stream))), "stencil_apply_region_put")


def stencil_slab_step_fused(plan: int, inputs: Sequence[int], out: int, put_lo: int = 0, put_hi: int = 0,
                            sig_lo: int = 0, sig_hi: int = 0, sig_value: int = 0, wait_lo: int = 0, wait_hi: int = 0,
                            wait_value: int = 0, stream: int = 0):
    v = lambda x: C.c_void_p(int(x)) if x else None
    _check(_slab_step_fused(plan, _ptrs(inputs), len(inputs), C.c_void_p(int(out)), v(put_lo), v(put_hi), v(sig_lo),
                            v(sig_hi), int(sig_value) & 0xffffffff, v(wait_lo), v(wait_hi),
                            int(wait_value) & 0xffffffff, C.c_void_p(int(stream))), "stencil_slab_step_fused")


def stencil_wait_signals(sig_a: int, sig_b: int, value: int, stream: int = 0):
    v = lambda x: C.c_void_p(int(x)) if x else None
    _check(_wait_signals(v(sig_a), v(sig_b), int(value) & 0xffffffff, C.c_void_p(int(stream))),
           "stencil_wait_signals")


def stencil_iterate(plan: int, state: Sequence[int], aux: Sequence[int], n_steps: int, stream: int = 0) -> int:
    ri = C.c_int32(-1)
    _check(_iterate(plan, _ptrs(state), len(state), _ptrs(aux), len(aux), int(n_steps), C.c_void_p(int(stream)),
                    C.byref(ri)), "stencil_iterate")
    return ri.value


def stencil_plan_last_kernel(plan: int) -> str:
    return _last_kernel(plan).decode()


def stencil_set_wait_timeout_ms(ms: int):
    _check(_set_wait_timeout(int(ms)), "stencil_set_wait_timeout_ms")


def stencil_device_fault():
    """Raises StencilError (E_CUDA) if a bounded halo wait timed out since the
    last check (call after synchronising the stream)."""
    _check(_device_fault(), "stencil_device_fault")


def stencil_run_host(plan: int, host_state: Sequence[np.ndarray], host_aux: Sequence[np.ndarray], n_steps: int,
                     host_out: np.ndarray, stream: int = 0):
    for a in list(host_state) + list(host_aux) + [host_out]:
        if a.dtype != np.float32 or not a.flags.c_contiguous:
            raise ValueError("host buffers must be C-contiguous float32")
    _check(_run_host(plan, _ptrs([a.ctypes.data for a in host_state]), len(host_state),
                     _ptrs([a.ctypes.data for a in host_aux]), len(host_aux), int(n_steps),
                     C.c_void_p(host_out.ctypes.data), C.c_void_p(int(stream))), "stencil_run_host")


def stencil_run_host_batch(plan: int, host_state: Sequence[np.ndarray], n_state: int,
                           host_aux: Sequence[np.ndarray], n_aux: int, n_steps: int, host_out: Sequence[np.ndarray]):
    """Jobs j = 0..len(host_out)-1: inputs host_state[j*n_state : (j+1)*n_state], aux host_aux[j*n_aux : ...]."""
    for a in list(host_state) + list(host_aux) + list(host_out):
        if a.dtype != np.float32 or not a.flags.c_contiguous:
            raise ValueError("host buffers must be C-contiguous float32")
    _check(_run_host_batch(plan, _ptrs([a.ctypes.data for a in host_state]), int(n_state),
                           _ptrs([a.ctypes.data for a in host_aux]), int(n_aux), int(n_steps), len(host_out),
                           _ptrs([a.ctypes.data for a in host_out])), "stencil_run_host_batch")


def stencil_plan_destroy(plan: int):
    _destroy(plan)
