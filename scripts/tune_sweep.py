"""Tuning sweep: run bench.py for (workload, env) combinations, print one line each.
usage: python scripts/tune_sweep.py 'workload:steps:ENV=V,ENV=V' ..."""
import json
import os
import subprocess
import sys

for spec in sys.argv[1:]:
    wl, steps, envs = (spec.split(":") + ["", ""])[:3]
    env = dict(os.environ)
    for kv in filter(None, envs.split(",")):
        k, v = kv.split("=")
        env[k] = v
    r = subprocess.run([sys.executable, "bench.py", "--workload", wl, "--no-cpu", "--no-e2e", "--steps", steps or "10"],
                       capture_output=True, text=True, env=env, timeout=600)
    try:
        d = json.loads(r.stdout.strip().splitlines()[-1])
        hot = (d.get("hot") or {}).get("value")
        print(f"{wl:26s} {envs:30s} {d['value']:8.1f} Gpts/s {d['roofline']['achieved']:7.0f} GB/s "
              f"frac {d['roofline']['frac']:.3f} of8 {d['roofline']['frac_of_8TBs']:.3f} "
              f"hot {'-' if hot is None else round(hot, 1)} sm {d['clocks']['sm_mhz']} "
              f"{','.join(d['clocks']['reasons'])} {d['config']['variant']}", flush=True)
    except Exception:
        print(wl, envs, "FAILED", r.stderr[-800:], flush=True)
