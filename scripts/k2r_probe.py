"""J3D7 512^3 x100: single-step K2 vs two steps per pass (K2R, registers) for
the K2R tile shapes / chunk knobs given on the command line, e.g.
    python scripts/k2r_probe.py 8: 6: 4: 8:16:4
(RPW:ZC:ZC2, empty = launcher default).  Timed with CUDA events, 100 steps
after 10 warm-up steps, best of 3."""
import os
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_cgo_hagedornssgd18_b200 as lift  # noqa: E402
import stencil_inputs as si  # noqa: E402

wl = os.environ.get("K2R_WORKLOAD", "j3d7_512_clamp")
scale = os.environ.get("K2R_SCALE")          # e.g. 128,128,128: override the extents
xs, spec = si.make_workload_inputs(si.workload(wl, scale=tuple(int(v) for v in scale.split(",")) if scale else None))
npts = 1
for e in spec.extents:
    npts *= e


def timed(tb, steps=100):
    plan = lift.Plan.from_spec(spec)
    plan.set_time_block(tb)
    a = torch.from_numpy(xs[0]).cuda()
    b = torch.empty_like(a)
    plan.iterate([a, b], 10)
    torch.cuda.synchronize()
    best = 1e9
    for _ in range(3):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        plan.iterate([a, b], steps)
        e1.record()
        torch.cuda.synchronize()
        best = min(best, e0.elapsed_time(e1) * 1e-3)
    return npts * steps / best / 1e9, plan.last_kernel


v, k = timed(1)
print(f"{wl} time_block 1: {v:7.1f} Gpts/s ({k})", flush=True)
for arg in sys.argv[1:] or ["8::"]:
    parts = (arg.split(":") + ["", "", ""])[:3]
    for key, val in zip(("LIFT_K2R_SHAPE", "LIFT_K2R_ZC", "LIFT_K2R_ZC2"), parts):
        if val:
            os.environ[key] = val
        else:
            os.environ.pop(key, None)
    v, k = timed(2)
    print(f"{wl} time_block 2 [{arg}]: {v:7.1f} Gpts/s ({k})", flush=True)
