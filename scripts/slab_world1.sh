#!/bin/bash
# The slab (multi-GPU) path at world size 1 (torchrun, one rank): halo path and depth
out=gpurun_out/slab_world1.txt; : > $out
run() {
  r=$(timeout 300 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 --master-addr 127.0.0.1 --master-port 29555 bench.py --gpus 1 --force-slab --steps 5 --warmup 3 --no-e2e --no-cpu "$@" 2>/dev/null | grep '^{' | tail -1)
  python - "$*" "$r" >> $out <<'PY'
import json, sys
a, r = sys.argv[1:]
try:
    d = json.loads(r)
    h = d.get("halo") or {}
    print(f"{a:52s} {d['value']:7.1f} Gpts/s  ms/step {d['ms_per_step']:.2f}  launches {d['gpu_launches']}  owned-sweep {h.get('owned_sweep_gpts', 0):.1f}")
except Exception:
    print(a, "ERR", r[:300])
PY
}
for d in 1 2 4 8; do run --halo-depth $d; done
run --halo fused
for d in 1 4; do run --workload acoustic13_1024 --scaling strong --halo-depth $d; done
run --workload acoustic13_1024 --scaling strong --halo fused
cat $out
