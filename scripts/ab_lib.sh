#!/bin/bash
# A/B of two in-tree library builds over workloads: ab_lib.sh OUT TAG_A TAG_B "wl1 wl2 ..." [rounds]
# (TAG "" = libstencil.so; other tags = libstencil_TAG.so, build.py with LIFT_LIB_TAG)
out=gpurun_out/$1; A=$2; B=$3; WLS=$4; R=${5:-2}
: > $out
for r in $(seq 1 $R); do
  for wl in $WLS; do
    for tag in "$A" "$B"; do
      res=$(LIFT_LIB_TAG=$tag timeout 300 python bench.py --workload $wl --steps 10 --warmup 3 --no-e2e --no-cpu 2>/dev/null | tail -1)
      python - "$tag" "$wl" "$res" >> $out <<'PY'
import json, sys
tag, wl, r = sys.argv[1:]
try:
    d = json.loads(r)
    hot = (d.get("hot") or {}).get("value")
    print(f"{wl:26s} lib={tag or 'main':8s} {d['value']:8.1f} Gpts/s  frac {d['roofline']['frac']:.3f}  hot {hot if hot is None else round(hot,1)}  sm {d['clocks']['sm_mhz']} {d['clocks']['reasons']}")
except Exception as e:
    print(wl, tag, "ERR", r[:200])
PY
    done
  done
done
cat $out
