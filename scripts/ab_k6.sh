#!/bin/bash
# A/B: Hotspot3D x100 on K6 (resident in shared memory) vs per-step K2C launches
out=gpurun_out/ab_k6.txt; : > $out
for cfg in "LIFT_K6=0" "LIFT_K6=1"; do
  for wl in hotspot3d_8x512x512_x100; do
    r=$(env $cfg timeout 120 python bench.py --workload $wl --steps 20 --warmup 5 --no-e2e --no-cpu 2>/dev/null | tail -1)
    python - "$cfg" "$wl" "$r" >> $out <<'PY'
import json, sys
cfg, wl, r = sys.argv[1:]
try:
    d = json.loads(r)
    hot = d.get("hot") or {}
    print(f"{wl:28s} {cfg:12s} cold {d['value']:7.1f}  hot {hot.get('value', float('nan')):7.1f} Gpts/s  frac {d['roofline']['frac']:.3f}  us/step {d['roofline']['avg_launch_us']:.2f} {d['config']['variant']}")
except Exception as e:
    print(wl, cfg, "ERR", r[:300])
PY
  done
done
cat $out
