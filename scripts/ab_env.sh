#!/bin/bash
# A/B of environment knobs on one workload: ab_env.sh OUT WORKLOAD "ENV1" "ENV2" ... (each "K=V K2=V2" or "-")
out=gpurun_out/$1; wl=$2; shift 2
: > $out
for r in 1 2; do
for cfg in "$@"; do
  e=""; [ "$cfg" != "-" ] && e="$cfg"
  res=$(env $e timeout 300 python bench.py --workload $wl --steps 10 --warmup 3 --no-e2e --no-cpu 2>/dev/null | tail -1)
  python - "$cfg" "$wl" "$res" >> $out <<'PY'
import json, sys
cfg, wl, r = sys.argv[1:]
try:
    d = json.loads(r)
    hot = (d.get("hot") or {}).get("value")
    print(f"{wl:24s} {cfg:28s} {d['value']:8.1f} Gpts/s  frac {d['roofline']['frac']:.3f} hot {hot if hot is None else round(hot,1)} sm {d['clocks']['sm_mhz']} {d['clocks']['reasons']}")
except Exception:
    print(wl, cfg, "ERR", r[:200])
PY
done
done
cat $out
