"""A few K2R passes on J3D7 512^3 (for ncu captures: -k regex:k2r)."""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_cgo_hagedornssgd18_b200 as lift  # noqa: E402
import stencil_inputs as si  # noqa: E402

xs, spec = si.make_workload_inputs(si.workload("j3d7_512_clamp"))
plan = lift.Plan.from_spec(spec)
plan.set_time_block(2)
a = torch.from_numpy(xs[0]).cuda()
b = torch.empty_like(a)
plan.iterate([a, b], 12)
torch.cuda.synchronize()
print(plan.last_kernel)
