"""K2 sweep bandwidth on a plain torch buffer vs a torch symmetric-memory
buffer (the fused slab path's state buffers), world size 1 (run under torchrun)."""
import os
import sys

import torch
import torch.distributed as dist
import torch.distributed._symmetric_memory as symm_mem

sys.path.insert(0, ".")
import stencil_inputs as si  # noqa: E402
import paper_conf_cgo_hagedornssgd18_b200 as lift  # noqa: E402

torch.cuda.set_device(0)
dist.init_process_group("nccl", device_id=torch.device("cuda:0"))
ext = (512, 512, 512)
sp = si.StencilSpec(ext, (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.CLAMP,) * 3, 0.0, si.WEIGHTED,
                    si.weights_j3d7(), ())
plan = lift.Plan.from_spec(sp)
x = torch.rand(ext, device="cuda")
for name, mk in [("plain", lambda: torch.empty(ext, device="cuda")),
                 ("symm", lambda: symm_mem.empty(*ext, dtype=torch.float32, device="cuda"))]:
    a, b = mk(), mk()
    if name == "symm":
        symm_mem.rendezvous(a, dist.group.WORLD)
        symm_mem.rendezvous(b, dist.group.WORLD)
    a.copy_(x)
    for _ in range(3):
        plan.iterate([a, b], 10)
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record()
    plan.iterate([a, b], 100)
    e1.record()
    torch.cuda.synchronize()
    t = e0.elapsed_time(e1) / 100
    print(f"{name}: {t * 1e3:.1f} us per step, {512 ** 3 / (t * 1e-3) / 1e9:.1f} Gpts/s", flush=True)
dist.destroy_process_group()

# the slab plan (ghost planes) of the fused bench path on both kinds of buffer
dist.init_process_group("nccl", device_id=torch.device("cuda:0"))
from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan, _NoExchange  # noqa: E402
s = SlabPlan(ext, 0, 1, size=3, kind="clamp", weights=si.weights_j3d7(), exchange=_NoExchange())
for name, mk in [("plain", lambda: torch.empty(s.alloc_shape, device="cuda")),
                 ("symm", lambda: symm_mem.empty(*s.alloc_shape, dtype=torch.float32, device="cuda"))]:
    a, b = mk(), mk()
    if name == "symm":
        symm_mem.rendezvous(a, dist.group.WORLD)
        symm_mem.rendezvous(b, dist.group.WORLD)
    a.copy_(torch.rand(s.alloc_shape, device="cuda"))
    for _ in range(3):
        s.plan.apply(a, out=b)
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record()
    for _ in range(50):
        s.plan.apply(a, out=b)
        s.plan.apply(b, out=a)
    e1.record()
    torch.cuda.synchronize()
    t = e0.elapsed_time(e1) / 100
    print(f"slab {name}: {t * 1e3:.1f} us per sweep, {512 ** 3 / (t * 1e-3) / 1e9:.1f} Gpts/s", flush=True)
dist.destroy_process_group()
