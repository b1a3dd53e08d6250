"""Acoustic 1024^3 x20: single steps (2 buffers) vs two steps per pass (K2RA,
4 buffers) for the shapes / chunk knobs on the command line, e.g.
    python scripts/k2ra_probe.py 7 6:: 4:: 4:32:8      (points, then RPW:ZC:ZC2)
Inputs: torch.rand on the device (the timing does not depend on values)."""
import os
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_cgo_hagedornssgd18_b200 as lift  # noqa: E402
import stencil_inputs as si  # noqa: E402

pts = int(sys.argv[1])
n = int(os.environ.get("K2RA_N", "1024"))
w = si.workload("acoustic7_1024" if pts == 7 else "acoustic13_1024")
spec = w.spec
spec.extents = (n, n, n)
bufs = [torch.rand((n, n, n), device="cuda") * 2 - 1 for _ in range(2)]
spare = [torch.empty_like(bufs[0]) for _ in range(2)]


def timed(nbuf, steps=20):
    plan = lift.Plan.from_spec(spec)
    plan.set_time_block(2 if nbuf == 4 else 1)
    st = bufs + (spare if nbuf == 4 else [])
    plan.iterate(st, 4)
    torch.cuda.synchronize()
    best = 1e9
    for _ in range(3):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        plan.iterate(st, steps)
        e1.record()
        torch.cuda.synchronize()
        best = min(best, e0.elapsed_time(e1) * 1e-3)
    return n ** 3 * steps / best / 1e9, plan.last_kernel


v, k = timed(2)
print(f"acoustic{pts} {n}^3 single steps: {v:7.1f} Gpts/s ({k})", flush=True)
if os.environ.get("K2RA_SINGLE_AGAIN"):
    v, k = timed(2)
    print(f"acoustic{pts} {n}^3 single steps (again): {v:7.1f} Gpts/s ({k})", flush=True)
for arg in sys.argv[2:] or ["::"]:
    parts = (arg.split(":") + ["", "", ""])[:3]
    for key, val in zip(("LIFT_K2RA_SHAPE", "LIFT_K2RA_ZC", "LIFT_K2RA_ZC2"), parts):
        if val:
            os.environ[key] = val
        else:
            os.environ.pop(key, None)
    v, k = timed(4)
    print(f"acoustic{pts} {n}^3 two steps [{arg}]: {v:7.1f} Gpts/s ({k})", flush=True)
