#!/bin/bash
# A/B of the Hotspot3D small-nz column shapes (LIFT_K2_HS) and z-chunks
out=gpurun_out/ab_hotspot.txt; : > $out
for hs in 0 1 2 3 4; do
  for zc in "" 8 4; do
    for wl in hotspot3d_8x512x512 hotspot3d_8x512x512_x100; do
      r=$(LIFT_K2_HS=$hs ${zc:+LIFT_K2_ZC=$zc} timeout 120 python bench.py --workload $wl --steps 20 --warmup 5 --no-e2e --no-cpu 2>/dev/null | tail -1)
      python - "$hs" "$zc" "$wl" "$r" >> $out <<'PY'
import json, sys
hs, zc, wl, r = sys.argv[1:]
try:
    d = json.loads(r)
    hot = d.get("hot") or {}
    print(f"{wl:28s} hs={hs} zc={zc or '-':3s} cold {d['value']:7.1f}  hot {hot.get('value', float('nan')):7.1f} Gpts/s  frac {d['roofline']['frac']:.3f} sm {d['clocks']['sm_mhz']}")
except Exception as e:
    print(wl, hs, zc, "ERR", r[:200])
PY
    done
  done
done
cat $out
