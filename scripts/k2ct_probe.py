"""Hotspot3D 8x512x512 x100 (L2-resident): single steps (K2C) vs two steps per
launch (K2CT) for the tile heights on the command line (LIFT_K2CT_TY), CUDA
graph of 100 steps replayed, best of 5."""
import os
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_cgo_hagedornssgd18_b200 as lift  # noqa: E402
import stencil_inputs as si  # noqa: E402

xs, spec = si.make_workload_inputs(si.workload("hotspot3d_8x512x512_x100"))
npts = 8 * 512 * 512


def timed(tb, steps=100):
    plan = lift.Plan.from_spec(spec)
    plan.set_time_block(tb)
    a = torch.from_numpy(xs[0]).cuda()
    b = torch.empty_like(a)
    pw = torch.from_numpy(xs[1]).cuda()
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        plan.iterate([a, b], steps, aux=[pw])
    torch.cuda.current_stream().wait_stream(s)
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        plan.iterate([a, b], steps, aux=[pw])
    g.replay()
    torch.cuda.synchronize()
    best = 1e9
    for _ in range(5):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        g.replay()
        e1.record()
        torch.cuda.synchronize()
        best = min(best, e0.elapsed_time(e1) * 1e-3)
    return npts * steps / best / 1e9, best / steps * 1e6, plan.last_kernel


v, us, k = timed(1)
print(f"hotspot3d x100 single steps: {v:7.1f} Gpts/s ({us:.2f} us/step, {k})", flush=True)
for ty in sys.argv[1:] or ["5"]:
    os.environ["LIFT_K2CT_TY"] = ty
    v, us, k = timed(2)
    print(f"hotspot3d x100 two steps per launch [TY={ty}]: {v:7.1f} Gpts/s ({us:.2f} us/step, {k})", flush=True)
