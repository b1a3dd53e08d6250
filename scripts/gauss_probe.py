"""Gaussian 8192^2: one cold sweep vs back-to-back sweeps (graph of 10), for
the library selected by LIFT_LIB_TAG."""
import os
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_cgo_hagedornssgd18_b200 as lift  # noqa: E402
import stencil_inputs as si  # noqa: E402

xs, spec = si.make_workload_inputs(si.workload("gauss5_8192_mirror"))
x = torch.from_numpy(xs[0]).cuda()
plan = lift.Plan.from_spec(spec)
out = plan.empty_output()
fb = torch.empty(63_000_000, dtype=torch.int32, device="cuda")
rb = torch.ones(63_000_000, dtype=torch.int32, device="cuda")
sink = torch.empty((), dtype=torch.int64, device="cuda")
ts = []
for k in range(13):
    fb.fill_(k)
    torch.sum(rb, 0, out=sink)
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    plan.apply(x, out=out)
    e1.record()
    torch.cuda.synchronize()
    if k >= 3:
        ts.append(e0.elapsed_time(e1) * 1e3)
ts.sort()
cold = ts[len(ts) // 2]
for mode in ("same", "pingpong"):
    y = torch.empty_like(out)
    g = torch.cuda.CUDAGraph()
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        plan.apply(x, out=out)
    torch.cuda.current_stream().wait_stream(s)
    with torch.cuda.graph(g):
        for i in range(10):
            if mode == "same":
                plan.apply(x, out=out)
            else:
                plan.apply(x if i % 2 == 0 else out, out=out if i % 2 == 0 else y)
    g.replay()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(5):
        g.replay()
    e1.record()
    torch.cuda.synchronize()
    t = e0.elapsed_time(e1) * 1e3 / 50
    print(f"lib={os.environ.get('LIFT_LIB_TAG', 'main'):7s} cold {cold:6.1f} us ({x.numel() / cold / 1e3:.0f} Gpts/s)  "
          f"back-to-back[{mode}] {t:6.1f} us ({x.numel() / t / 1e3:.0f} Gpts/s)")
