"""The C ABI used from plain C (examples/c_abi_demo.c, no Python/torch in the
process): build with gcc against include/stencil.h, run on the GPU, compare
its outputs with the fp64 oracle."""
import os
import shutil
import subprocess

import numpy as np
import pytest

import stencil_inputs as si
from oracle import stencil_oracle as orc

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def test_c_program_parity(tmp_path):
    import __graft_entry__
    __graft_entry__.build()
    pkg = os.path.join(ROOT, "paper_conf_cgo_hagedornssgd18_b200")
    exe = tmp_path / "c_abi_demo"
    subprocess.run(["gcc", "-O2", "-std=c99", "-I", os.path.join(ROOT, "include"),
                    os.path.join(ROOT, "examples", "c_abi_demo.c"), "-L", pkg, "-lstencil",
                    "-L/usr/local/cuda/lib64", "-lcudart", f"-Wl,-rpath,{pkg}", "-o", str(exe)], check=True)
    r = subprocess.run([str(exe), "it.f32", "ap.f32"], cwd=tmp_path, capture_output=True, text=True, timeout=120)
    assert r.returncode == 0, r.stdout + r.stderr
    assert "variant 2" in r.stdout          # the TMA sweep kernel ran
    ext = (20, 36, 132)
    x = np.fromfile(tmp_path / "c_abi_demo_input.f32", np.float32).reshape(ext)
    w = si.weights_j3d7()
    sp = si.StencilSpec(ext, (3, 3, 3), (1, 1, 1), (1, 1, 1), (1, 1, 1), (si.CLAMP, si.MIRROR, si.WRAP), 0.0,
                        si.WEIGHTED, w, ())
    Y, A = orc.apply(sp, [x])
    ap = np.fromfile(tmp_path / "ap.f32", np.float32).reshape(ext)
    assert orc.max_rel_err(ap, Y, A) <= 1e-5
    it = np.fromfile(tmp_path / "it.f32", np.float32).reshape(ext)
    ref = orc.iterate(sp, [x], [], 3)[0]
    assert np.max(np.abs(it - ref) / np.abs(ref)) <= 1e-4
