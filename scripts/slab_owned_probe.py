"""Owned-slab sweep timing before / after a deep-halo SlabPlan.iterate (world 1)."""
import sys

import torch

sys.path.insert(0, ".")
import stencil_inputs as si  # noqa: E402
from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan, _NoExchange  # noqa: E402


def t_apply(s, a, b, n=20):
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(n):
        s.plan.apply(a, out=b)
    e1.record()
    torch.cuda.synchronize()
    return 512 ** 3 / (e0.elapsed_time(e1) * 1e-3 / n) / 1e9, s.plan.last_kernel


for depth in (1, 4):
    s = SlabPlan((512, 512, 512), 0, 1, size=3, kind="clamp", weights=si.weights_j3d7(), exchange=_NoExchange(),
                 depth=depth)
    a = s.empty().uniform_(0.5, 1.5)
    b = s.empty()
    print("depth", depth, "before", t_apply(s, a, b), flush=True)
    ri = s.iterate([a, b], 100)
    print("depth", depth, "after iterate (ri=%d)" % ri, t_apply(s, a, b), t_apply(s, (a, b)[ri], (a, b)[1 - ri]),
          flush=True)
