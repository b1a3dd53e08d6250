#!/bin/bash
python scripts/k2t_probe.py
cat > /tmp/k2tone.py <<'PY'
import sys, torch
sys.path.insert(0, ".")
import paper_conf_cgo_hagedornssgd18_b200 as lift
import stencil_inputs as si
xs, spec = si.make_workload_inputs(si.workload("j3d7_512_clamp"))
plan = lift.Plan.from_spec(spec); plan.set_time_block(2)
a = torch.from_numpy(xs[0]).cuda(); b = torch.empty_like(a)
plan.iterate([a, b], 8); torch.cuda.synchronize()
PY
timeout 600 ncu --set full --clock-control none --import-source on -k "regex:k2t" --launch-skip 2 --launch-count 1 -o gpurun_out/ncu_k2t -f python /tmp/k2tone.py > /dev/null 2>&1
python scripts/ncu_summary.py gpurun_out/ncu_k2t.ncu-rep | head -19
python scripts/op_hist.py gpurun_out/ncu_k2t.ncu-rep | head -26
ncu -i gpurun_out/ncu_k2t.ncu-rep --page source --csv --print-source sass > gpurun_out/k2t_src.csv 2>/dev/null
rm -f gpurun_out/*.ncu-rep
