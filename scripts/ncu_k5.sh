#!/bin/bash
# strided K5 throughput + one ncu --set full capture of the 512^3 3x3x3 step-2 launch
python scripts/strided_probe.py 2>&1 | tail -5
cat > /tmp/k5one.py <<'PY'
import sys, torch, numpy as np
sys.path.insert(0, ".")
import stencil_inputs as si
import paper_conf_cgo_hagedornssgd18_b200 as lift
ext = (512, 512, 512)
w = np.full((3, 3, 3), 1.0 / 27, np.float32)
sp = si.StencilSpec(ext, (3,) * 3, (2,) * 3, (1,) * 3, (1,) * 3, (si.CLAMP,) * 3, 0.0, si.WEIGHTED, w, ())
plan = lift.Plan.from_spec(sp)
x = torch.rand(ext, device="cuda")
y = plan.apply(x)
for _ in range(4):
    plan.apply(x, out=y)
torch.cuda.synchronize()
PY
timeout 600 ncu --set full --clock-control none --import-source on -k "regex:k5" --launch-skip 2 --launch-count 1 -o gpurun_out/ncu_r02_k5_3d -f python /tmp/k5one.py > /dev/null 2>&1
python scripts/ncu_summary.py gpurun_out/ncu_r02_k5_3d.ncu-rep 2>&1 | head -20
python scripts/op_hist.py gpurun_out/ncu_r02_k5_3d.ncu-rep 2>&1 | head -16
python scripts/stall_top.py gpurun_out/ncu_r02_k5_3d.ncu-rep 15 2>&1 | tail -17
rm -f gpurun_out/*.ncu-rep
