#!/bin/bash
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
timeout 600 ncu --set full --clock-control none --import-source on -k "regex:k5" --launch-skip 2 --launch-count 1 -o gpurun_out/ncu_k5src -f python /tmp/k5one.py > /dev/null 2>&1
ncu -i gpurun_out/ncu_k5src.ncu-rep --page source --csv --print-source sass > gpurun_out/k5_src.csv 2>/dev/null
ncu -i gpurun_out/ncu_k5src.ncu-rep --page source --csv --print-source cuda > gpurun_out/k5_cuda.csv 2>/dev/null
rm -f gpurun_out/*.ncu-rep
