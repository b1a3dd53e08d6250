"""Torch-facing convenience layer over the C ABI (device memory and streams
only — PyTorch is plumbing here; all stencil work runs in libstencil.so).

    plan = Plan(extents=(512, 512, 512), size=3, pad=1, kind="clamp",
                op="weighted", weights=w)
    y = plan.apply(x)                      # x: contiguous fp32 CUDA tensor
    idx = plan.iterate([x, scratch], n_steps=100)
"""
from __future__ import annotations

from typing import Optional, Sequence, Union

import numpy as np
import torch

from . import _lib as L

KINDS = {"clamp": L.PAD_CLAMP, "mirror": L.PAD_MIRROR, "symmetric": L.PAD_MIRROR, "wrap": L.PAD_WRAP,
         "constant": L.PAD_CONSTANT, "zero": L.PAD_CONSTANT, "reflect": L.PAD_REFLECT, "dampen": L.PAD_DAMPEN}
OPS = {"weighted": L.OP_WEIGHTED, "hotspot3d": L.OP_HOTSPOT3D, "srad1": L.OP_SRAD1, "srad2": L.OP_SRAD2,
       "acoustic": L.OP_ACOUSTIC, "hotspot2d": L.OP_HOTSPOT2D, "gradient": L.OP_GRADIENT,
       "srad": L.OP_SRAD}
VARIANTS = {"auto": L.VARIANT_AUTO, "generic": L.VARIANT_GENERIC, "tile2d": L.VARIANT_TILE2D,
            "sweep3d": L.VARIANT_SWEEP3D, "persist3d": L.VARIANT_PERSIST3D,
            "gather": L.VARIANT_GATHER, "resident3d": L.VARIANT_RESIDENT3D}


def _tuple(v, nd):
    if isinstance(v, (list, tuple)):
        assert len(v) == nd
        return tuple(int(x) for x in v)
    return (int(v),) * nd


def _kind(k):
    return KINDS[k] if isinstance(k, str) else int(k)


def _stream_handle(stream: Optional[torch.cuda.Stream]) -> int:
    s = stream if stream is not None else torch.cuda.current_stream()
    return int(s.cuda_stream)


class Plan:
    """map_n(f, slide_n(size, step, pad_n(l, r, h, input)))."""

    def __init__(self, extents: Sequence[int], size: Union[int, Sequence[int]] = 3,
                 step: Union[int, Sequence[int]] = 1, pad: Union[None, int, Sequence[int]] = None,
                 pad_hi: Union[None, int, Sequence[int]] = None, kind="clamp", pad_value: float = 0.0,
                 op="weighted", weights=None, params: Sequence[float] = (), device: Optional[int] = None):
        nd = len(extents)
        self.ndim = nd
        self.extents = tuple(int(e) for e in extents)
        self.size = _tuple(size, nd)
        self.step = _tuple(step, nd)
        self.pad_lo = tuple(s // 2 for s in self.size) if pad is None else _tuple(pad, nd)
        self.pad_hi = self.pad_lo if pad_hi is None and pad is not None else (
            tuple(s - 1 - l for s, l in zip(self.size, self.pad_lo)) if pad_hi is None else _tuple(pad_hi, nd))
        kinds = kind if isinstance(kind, (list, tuple)) else [kind] * nd
        self.kind = tuple(_kind(k) for k in kinds)
        self.pad_value = float(pad_value)
        self.op = OPS[op] if isinstance(op, str) else int(op)
        self.weights = None if weights is None else np.asarray(weights, np.float32)
        self.params = tuple(float(p) for p in params)
        self.device = torch.cuda.current_device() if device is None else int(device)
        self.handle = L.stencil_plan_create(self.device, self.extents, self.size, self.step, self.pad_lo,
                                            self.pad_hi, self.kind, self.pad_value, self.op, self.weights,
                                            self.params)
        self.out_extents = L.stencil_plan_output_extents(self.handle, nd)
        self.ghost = 0
        self.alloc_extents = self.extents
        self.out_alloc_extents = self.out_extents

    @classmethod
    def from_spec(cls, spec, device: Optional[int] = None) -> "Plan":
        """Build from a stencil_inputs.StencilSpec-like object (duck-typed)."""
        plan = cls(spec.extents, spec.size, spec.step, spec.pad_lo, spec.pad_hi, list(spec.kind),
                   spec.pad_value, spec.op, spec.weights, spec.params, device)
        decay = getattr(spec, "pad_decay", 1.0)
        if decay != 1.0:
            plan.set_pad_decay(decay)
        return plan

    def set_pad_decay(self, decay: float):
        """DAMPEN dimensions: factor per cell of distance outside the grid (A29)."""
        L.stencil_plan_set_pad_decay(self.handle, decay)

    def set_slab(self, z_offset: int, global_n0: int, ghost: int):
        L.stencil_plan_set_slab(self.handle, z_offset, global_n0, ghost)
        self.ghost = int(ghost)
        self.alloc_extents = (self.extents[0] + 2 * ghost,) + self.extents[1:]
        self.out_alloc_extents = self.alloc_extents

    def set_variant(self, variant):
        L.stencil_plan_set_variant(self.handle, VARIANTS[variant] if isinstance(variant, str) else int(variant))

    def set_time_block(self, steps: int):
        L.stencil_plan_set_time_block(self.handle, steps)

    @property
    def time_block(self) -> int:
        return L.stencil_plan_time_block(self.handle)

    @property
    def variant(self) -> int:
        return L.stencil_plan_variant(self.handle)

    @property
    def last_kernel(self) -> str:
        """Kernel function of the most recent launch (e.g. 'k2_sweep', 'k2c_column')."""
        return L.stencil_plan_last_kernel(self.handle)

    @property
    def last_variant(self) -> int:
        """Kernel family of the most recent apply / iterate launch."""
        return L.stencil_plan_last_variant(self.handle)

    def _check(self, t: torch.Tensor, shape, name):
        if not isinstance(t, torch.Tensor) or not t.is_cuda:
            raise TypeError(f"{name} must be a CUDA tensor (no CPU fallback)")
        if t.dtype != torch.float32 or not t.is_contiguous():
            raise TypeError(f"{name} must be contiguous float32")
        if tuple(t.shape) != tuple(shape):
            raise ValueError(f"{name} has shape {tuple(t.shape)}, expected {tuple(shape)}")

    def empty_output(self) -> torch.Tensor:
        return torch.empty(self.out_alloc_extents, dtype=torch.float32, device=f"cuda:{self.device}")

    def apply(self, *inputs: torch.Tensor, out: Optional[torch.Tensor] = None,
              stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
        for i, x in enumerate(inputs):
            self._check(x, self.alloc_extents, f"input {i}")
        if out is None:
            out = self.empty_output()
        self._check(out, self.out_alloc_extents, "out")
        L.stencil_apply(self.handle, [x.data_ptr() for x in inputs], out.data_ptr(), _stream_handle(stream))
        return out

    def apply_region(self, *inputs: torch.Tensor, out: torch.Tensor, begin: int, end: int,
                     stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
        for i, x in enumerate(inputs):
            self._check(x, self.alloc_extents, f"input {i}")
        self._check(out, self.out_alloc_extents, "out")
        L.stencil_apply_region(self.handle, [x.data_ptr() for x in inputs], out.data_ptr(), begin, end,
                               _stream_handle(stream))
        return out

    def apply2_region(self, x: torch.Tensor, out: torch.Tensor, begin: int, end: int,
                      stream: Optional[torch.cuda.Stream] = None) -> torch.Tensor:
        """Two time steps in one pass on output planes [begin, end) (stencil_apply2_region)."""
        self._check(x, self.alloc_extents, "input")
        self._check(out, self.out_alloc_extents, "out")
        L.stencil_apply2_region(self.handle, x.data_ptr(), out.data_ptr(), begin, end, _stream_handle(stream))
        return out

    def iterate(self, state: Sequence[torch.Tensor], n_steps: int, aux: Sequence[torch.Tensor] = (),
                stream: Optional[torch.cuda.Stream] = None) -> int:
        for i, x in enumerate(list(state) + list(aux)):
            self._check(x, self.alloc_extents, f"state/aux {i}")
        return L.stencil_iterate(self.handle, [x.data_ptr() for x in state], [x.data_ptr() for x in aux],
                                 n_steps, _stream_handle(stream))

    def run_host(self, host_state: Sequence[np.ndarray], n_steps: int = 1,
                 host_aux: Sequence[np.ndarray] = (), out: Optional[np.ndarray] = None,
                 stream: Optional[torch.cuda.Stream] = None) -> np.ndarray:
        if out is None:
            out = np.empty(self.out_alloc_extents, np.float32)
        # the C side copies whole grids: a wrongly sized host array would be
        # over-read / over-written, so check every size here
        n_in = int(np.prod(self.alloc_extents))
        for a in list(host_state) + list(host_aux):
            if np.asarray(a).size != n_in:
                raise ValueError(f"run_host: input of {np.asarray(a).size} elements, plan needs {n_in}")
        if out.size != int(np.prod(self.out_alloc_extents)):
            raise ValueError(f"run_host: out has {out.size} elements, plan writes {int(np.prod(self.out_alloc_extents))}")
        L.stencil_run_host(self.handle, list(host_state), list(host_aux), n_steps, out, _stream_handle(stream))
        return out

    def run_host_batch(self, jobs: Sequence[Sequence[np.ndarray]], n_steps: int = 1,
                       aux: Sequence[Sequence[np.ndarray]] = (), outs: Optional[Sequence[np.ndarray]] = None):
        """Independent jobs (each a list of host state grids, plus its aux grids)
        with copy-in / compute / copy-out overlapped across jobs
        (stencil_run_host_batch); returns the list of output arrays."""
        n_in = int(np.prod(self.alloc_extents))
        n_out = int(np.prod(self.out_alloc_extents))
        if outs is None:
            outs = [np.empty(self.out_alloc_extents, np.float32) for _ in jobs]
        if len(outs) != len(jobs) or (aux and len(aux) != len(jobs)):
            raise ValueError("run_host_batch: one output (and aux list) per job")
        n_state = len(jobs[0])
        n_aux = len(aux[0]) if aux else 0
        flat, flat_aux = [], []
        for j, st in enumerate(jobs):
            if len(st) != n_state or (aux and len(aux[j]) != n_aux):
                raise ValueError("run_host_batch: every job needs the same number of grids")
            for a in list(st) + (list(aux[j]) if aux else []):
                if np.asarray(a).size != n_in:
                    raise ValueError(f"run_host_batch: input of {np.asarray(a).size} elements, plan needs {n_in}")
            flat += list(st)
            flat_aux += list(aux[j]) if aux else []
        for o in outs:
            if o.size != n_out:
                raise ValueError(f"run_host_batch: out has {o.size} elements, plan writes {n_out}")
        L.stencil_run_host_batch(self.handle, flat, n_state, flat_aux, n_aux, n_steps, list(outs))
        return list(outs)

    def close(self):
        if getattr(self, "handle", None):
            L.stencil_plan_destroy(self.handle)
            self.handle = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass
