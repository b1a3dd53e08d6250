"""Build libstencil.so in-tree with nvcc for sm_100a (no JIT, no torch extension).

    python paper_conf_cgo_hagedornssgd18_b200/build.py [-v] [-f]

(run it as a script, or through __graft_entry__.build(): importing it via the
package would load libstencil.so before it exists)

Every .cu under csrc/ is compiled separately (in parallel) and linked into
``paper_conf_cgo_hagedornssgd18_b200/libstencil.so`` with a static CUDA
runtime.  ``-fmad=false``: the only fused multiply-adds are the explicit
``__fmaf_rn`` of ops.cuh, so every kernel family rounds identically
(reading A12/A24).
"""
from __future__ import annotations

import concurrent.futures as cf
import glob
import os
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
# LIFT_LIB_TAG=x builds an A/B variant libstencil_x.so (objects in _build_x)
# with the extra nvcc flags of LIFT_NVCC_EXTRA (e.g. -DLIFT_MBAR_SPIN); the
# binding loads it with the same variable
_TAG = os.environ.get("LIFT_LIB_TAG", "")
BUILD = os.path.join(PKG, f"_build_{_TAG}" if _TAG else "_build")
LIB = os.path.join(PKG, f"libstencil_{_TAG}.so" if _TAG else "libstencil.so")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")

ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]
CFLAGS = ["-O3", "-std=c++17", "-lineinfo", "-fmad=false", "-Xcompiler", "-fPIC",
          "-Xcompiler", "-Wall", "-I" + os.path.join(ROOT, "include"), "-I" + CSRC,
          "--expt-relaxed-constexpr"] + os.environ.get("LIFT_NVCC_EXTRA", "").split()


def _sources():
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")))


def _headers():
    return sorted(glob.glob(os.path.join(CSRC, "*.cuh")) + glob.glob(os.path.join(CSRC, "*.hpp")) +
                  glob.glob(os.path.join(ROOT, "include", "*.h")))


def _stale(target, deps):
    if not os.path.exists(target):
        return True
    t = os.path.getmtime(target)
    return any(os.path.getmtime(d) > t for d in deps)


def _compile(src, verbose):
    obj = os.path.join(BUILD, os.path.basename(src) + ".o")
    if not _stale(obj, [src] + _headers() + [__file__]):
        return obj, ""
    cmd = [NVCC] + ARCH + CFLAGS + ["-Xptxas", "-v", "-c", src, "-o", obj]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError(f"nvcc failed for {src}:\n{' '.join(cmd)}\n{r.stdout}\n{r.stderr}")
    return obj, (r.stdout + r.stderr) if verbose else ""


def build(verbose: bool = False, force: bool = False) -> str:
    os.makedirs(BUILD, exist_ok=True)
    srcs = _sources()
    if force:
        for o in glob.glob(os.path.join(BUILD, "*.o")):
            os.remove(o)
    with cf.ThreadPoolExecutor(max_workers=min(8, os.cpu_count() or 4)) as ex:
        results = list(ex.map(lambda s: _compile(s, verbose), srcs))
    objs = [o for o, _ in results]
    if verbose:
        for _, log in results:
            if log:
                print(log)
    if force or _stale(LIB, objs):
        cmd = [NVCC] + ARCH + ["-shared", "-cudart", "static", "-o", LIB] + objs
        r = subprocess.run(cmd, capture_output=True, text=True)
        if r.returncode != 0:
            raise RuntimeError(f"link failed:\n{' '.join(cmd)}\n{r.stdout}\n{r.stderr}")
    return LIB


if __name__ == "__main__":
    print(build(verbose="-v" in sys.argv, force="-f" in sys.argv))
