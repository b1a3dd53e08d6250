"""J3D7 512^3 x100: single-step K2 vs the two-step K2T (stencil_plan_set_time_block(2))."""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_cgo_hagedornssgd18_b200 as lift  # noqa: E402
import stencil_inputs as si  # noqa: E402

xs, spec = si.make_workload_inputs(si.workload("j3d7_512_clamp"))
for tb in (1, 2):
    plan = lift.Plan.from_spec(spec)
    plan.set_time_block(tb)
    a = torch.from_numpy(xs[0]).cuda()
    b = torch.empty_like(a)
    plan.iterate([a, b], 10)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    plan.iterate([a, b], 100)
    e1.record()
    torch.cuda.synchronize()
    t = e0.elapsed_time(e1) * 1e-3
    print(f"time_block {tb}: {512 ** 3 * 100 / t / 1e9:7.1f} Gpts/s  ({t * 1e3 / 100 * 1e3:.1f} us per step)", flush=True)
