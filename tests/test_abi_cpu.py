"""C-ABI library checks that need no GPU: the library loads, exports every
symbol include/stencil.h declares, and validates plans on the host (the
pad/slide types of PAPER.md P:416-422).  No compute calls."""
import ctypes
import os
import re

import numpy as np
import pytest

import stencil_inputs as si
from oracle.stencil_oracle import slide_count

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "stencil.h")


@pytest.fixture(scope="module")
def lib():
    import __graft_entry__
    __graft_entry__.build()
    import paper_conf_cgo_hagedornssgd18_b200 as m
    return m


def declared_symbols():
    txt = open(HEADER).read()
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    return sorted(set(re.findall(r"\b(stencil_[a-z0-9_]+)\s*\(", txt)))


def test_header_symbols_exported(lib):
    so = ctypes.CDLL(lib._lib.LIB_PATH)
    syms = declared_symbols()
    assert len(syms) >= 12
    for s in syms:
        assert hasattr(so, s), f"{s} declared in stencil.h but not exported"
    assert set(syms) == set(lib._lib.EXPORTED)


def test_binding_names_match_abi(lib):
    for s in declared_symbols():
        assert callable(getattr(lib, s)), s


def test_library_is_sm100a():
    import subprocess
    so = os.path.join(ROOT, "paper_conf_cgo_hagedornssgd18_b200", "libstencil.so")
    r = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "--list-elf", so], capture_output=True, text=True)
    assert "sm_100a" in r.stdout


def test_output_extents_match_slide_count(lib):
    rng = np.random.default_rng(0)
    for _ in range(50):
        nd = int(rng.integers(1, 4))
        ext = [int(rng.integers(1, 40)) for _ in range(nd)]
        size = [int(rng.integers(1, 6)) for _ in range(nd)]
        step = [int(rng.integers(1, 4)) for _ in range(nd)]
        lo = [int(rng.integers(0, 4)) for _ in range(nd)]
        hi = [int(rng.integers(0, 4)) for _ in range(nd)]
        if any(n + l + r < s for n, l, r, s in zip(ext, lo, hi, size)):
            with pytest.raises(lib.StencilError) as e:
                lib.stencil_plan_create(0, ext, size, step, lo, hi, [0] * nd, 0.0, 0, np.ones(size, np.float32))
            assert e.value.status == 1
            continue
        h = lib.stencil_plan_create(0, ext, size, step, lo, hi, [0] * nd, 0.0, 0, np.ones(size, np.float32))
        got = lib.stencil_plan_output_extents(h, nd)
        exp = tuple(slide_count(n + l + r, s, st) for n, l, r, s, st in zip(ext, lo, hi, size, step))
        assert got == exp
        lib.stencil_plan_destroy(h)


@pytest.mark.parametrize("bad", [
    dict(ext=[0, 4]), dict(size=[0, 3]), dict(step=[1, 0]), dict(lo=[-1, 1]), dict(kind=[0, 9]),
    dict(ext=[1, 1], lo=[0, 0], hi=[0, 0]),      # n + l + r < size
    dict(weights=None), dict(op=7),
])
def test_plan_validation_invalid(lib, bad):
    args = dict(ext=[8, 8], size=[3, 3], step=[1, 1], lo=[1, 1], hi=[1, 1], kind=[0, 0], op=0,
                weights=np.ones((3, 3), np.float32))
    args.update(bad)
    with pytest.raises(lib.StencilError) as e:
        lib.stencil_plan_create(0, args["ext"], args["size"], args["step"], args["lo"], args["hi"], args["kind"],
                                0.0, args["op"], args["weights"])
    assert e.value.status == 1


def test_plan_validation_op_shapes(lib):
    # HOTSPOT3D must be 3D size 3 pad 1
    with pytest.raises(lib.StencilError):
        lib.stencil_plan_create(0, [8, 8], [3, 3], [1, 1], [1, 1], [1, 1], [0, 0], 0.0, si.HOTSPOT3D, None,
                                si.params_hotspot3d())
    # SRAD must be 2D
    with pytest.raises(lib.StencilError):
        lib.stencil_plan_create(0, [4, 8, 8], [3] * 3, [1] * 3, [1] * 3, [1] * 3, [0] * 3, 0.0, si.SRAD1, None, (0.1,))
    # acoustic with size 5 pad 2 is fine
    h = lib.stencil_plan_create(0, [8, 8, 8], [5] * 3, [1] * 3, [2] * 3, [2] * 3, [3] * 3, 0.0, si.ACOUSTIC, None,
                                si.params_acoustic(13))
    lib.stencil_plan_destroy(h)


def test_too_many_taps_unsupported(lib):
    with pytest.raises(lib.StencilError) as e:
        lib.stencil_plan_create(0, [20, 20, 20], [6, 6, 6], [1] * 3, [2] * 3, [3] * 3, [0] * 3, 0.0, 0,
                                np.ones((6, 6, 6), np.float32))
    assert e.value.status == 2


def test_ndim4_unsupported(lib):
    with pytest.raises(lib.StencilError) as e:
        lib.stencil_plan_create(0, [2] * 4, [1] * 4, [1] * 4, [0] * 4, [0] * 4, [0] * 4, 0.0, 0, np.ones(1, np.float32))
    assert e.value.status == 2


def test_slab_validation(lib):
    h = lib.stencil_plan_create(0, [16, 8, 8], [3] * 3, [1] * 3, [1] * 3, [1] * 3, [0] * 3, 0.0, 0,
                                si.weights_j3d7())
    lib.stencil_plan_set_slab(h, 16, 64, 1)
    with pytest.raises(lib.StencilError):
        lib.stencil_plan_set_slab(h, 60, 64, 1)     # slab outside the grid
    with pytest.raises(lib.StencilError):
        lib.stencil_plan_set_slab(h, 0, 64, 0)      # ghost < pad
    lib.stencil_plan_destroy(h)


def test_product_package_does_not_import_oracle():
    pkg = os.path.join(ROOT, "paper_conf_cgo_hagedornssgd18_b200")
    pat = re.compile(r"^\s*(import|from)\s+(\.\.)?oracle\b|#include\s+.*oracle", re.M)
    for dirpath, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".hpp", ".cpp", ".h")):
                txt = open(os.path.join(dirpath, f)).read()
                assert not pat.search(txt), f


def test_dampen_pad_validation(lib):
    """DAMPEN (reading A29) is a WEIGHTED pad kind; its decay lies in [0, 1]."""
    with pytest.raises(lib.StencilError) as e:
        lib.stencil_plan_create(0, [8, 8], [3, 3], [1, 1], [1, 1], [1, 1], [si.DAMPEN, 0], 0.0, si.SRAD1, None, (0.1,))
    assert e.value.status == 2
    with pytest.raises(lib.StencilError) as e:
        lib.stencil_plan_create(0, [8, 8], [3, 3], [1, 1], [1, 1], [1, 1], [6, 0], 0.0, 0, np.ones((3, 3), np.float32))
    assert e.value.status == 1
    h = lib.stencil_plan_create(0, [8, 8], [3, 3], [1, 1], [1, 1], [1, 1], [si.DAMPEN, si.DAMPEN], 0.0, 0,
                                np.ones((3, 3), np.float32))
    lib.stencil_plan_set_pad_decay(h, 0.25)
    for bad in (-0.1, 1.5, float("nan")):
        with pytest.raises(lib.StencilError):
            lib.stencil_plan_set_pad_decay(h, bad)
    # DAMPEN plans never take the TMA families
    assert lib.stencil_plan_variant(h) == lib._lib.VARIANT_GATHER
    lib.stencil_plan_destroy(h)
