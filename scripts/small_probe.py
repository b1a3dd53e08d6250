"""Cold single sweeps of the small BASELINE grids per kernel family (K1 tile
vs K0 generic): J2D5 256^2, SRAD1 504x458, Hotspot3D 8x512x512."""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_cgo_hagedornssgd18_b200 as lift  # noqa: E402
import stencil_inputs as si  # noqa: E402

L2 = 126_000_000
fb = torch.empty(int(2 * L2) // 4, dtype=torch.int32, device="cuda")
rb = torch.ones(int(2 * L2) // 4, dtype=torch.int32, device="cuda")
sink = torch.empty((), dtype=torch.int64, device="cuda")


def cold(fn, reps=30):
    ts = []
    for k in range(reps + 3):
        fb.fill_(k)
        torch.sum(rb, 0, out=sink)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        fn()
        e1.record()
        torch.cuda.synchronize()
        if k >= 3:
            ts.append(e0.elapsed_time(e1) * 1e3)
    ts.sort()
    return ts[len(ts) // 2]


for wl in ["j2d5_256_clamp", "t1_srad1_504x458", "hotspot3d_8x512x512"]:
    xs, spec = si.make_workload_inputs(si.workload(wl))
    dev = [torch.from_numpy(x).cuda() for x in xs]
    for var in ["auto", "generic"]:
        plan = lift.Plan.from_spec(spec)
        plan.set_variant(var)
        out = plan.empty_output()
        us = cold(lambda: plan.apply(*dev, out=out))
        npts = out.numel()
        print(f"{wl:22s} {var:8s} {us:7.2f} us  {npts / us / 1e3:7.1f} Gpts/s  last_variant {plan.last_variant}")
