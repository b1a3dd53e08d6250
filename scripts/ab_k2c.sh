#!/bin/bash
# A/B: Hotspot3D (8,512,512) on K2C (tile rows 4 / 8) vs the K2 ring (LIFT_K2C=0)
out=gpurun_out/ab_k2c.txt; : > $out
for cfg in "LIFT_K2C=0" "LIFT_K2C_TY=4" "LIFT_K2C_TY=8"; do
  for wl in hotspot3d_8x512x512 hotspot3d_8x512x512_x100; do
    r=$(env $cfg timeout 120 python bench.py --workload $wl --steps 20 --warmup 5 --no-e2e --no-cpu 2>/dev/null | tail -1)
    python - "$cfg" "$wl" "$r" >> $out <<'PY'
import json, sys
cfg, wl, r = sys.argv[1:]
try:
    d = json.loads(r)
    hot = d.get("hot") or {}
    print(f"{wl:28s} {cfg:16s} cold {d['value']:7.1f}  hot {hot.get('value', float('nan')):7.1f} Gpts/s  frac {d['roofline']['frac']:.3f}  us/launch {d['roofline']['avg_launch_us']:.2f}")
except Exception as e:
    print(wl, cfg, "ERR", r[:300])
PY
  done
done
cat $out
