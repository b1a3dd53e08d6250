"""Throughput of strided slides (step > 1, NEXT-4) on the generic kernel K0:
output points/s and input+output bytes/s for a few downsampling shapes."""
import sys
import torch
sys.path.insert(0, ".")
import numpy as np
import stencil_inputs as si
import paper_conf_cgo_hagedornssgd18_b200 as lift

cases = [((8192, 8192), 3, 2), ((8192, 8192), 5, 2), ((8192, 8192), 2, 2), ((512, 512, 512), 3, 2), ((512, 512, 512), 2, 2)]
for ext, size, step in cases:
    nd = len(ext)
    w = np.full((size,) * nd, 1.0 / size ** nd, np.float32)
    lo = tuple([size // 2] * nd) if size % 2 else tuple([0] * nd)
    hi = tuple([size // 2] * nd) if size % 2 else tuple([size - 1] * nd)
    sp = si.StencilSpec(ext, (size,) * nd, (step,) * nd, lo, hi, (si.CLAMP,) * nd, 0.0, si.WEIGHTED, w, ())
    plan = lift.Plan.from_spec(sp)
    x = torch.rand(ext, device="cuda")
    y = plan.apply(x)
    for _ in range(3):
        plan.apply(x, out=y)
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record()
    n = 10
    for _ in range(n):
        plan.apply(x, out=y)
    e1.record()
    torch.cuda.synchronize()
    t = e0.elapsed_time(e1) / n * 1e-3
    pts = y.numel()
    byts = (x.numel() + y.numel()) * 4
    print(f"{str(ext):18s} size {size} step {step} variant {plan.variant}: {pts / t / 1e9:7.1f} Gpts/s  "
          f"{byts / t / 1e9:7.0f} GB/s (in+out)  {t * 1e6:8.1f} us", flush=True)
