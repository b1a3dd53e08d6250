#!/bin/bash
for e in 0 1 0 1; do
  r=$(LIFT_FUSED_PDL=$e timeout 300 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 --master-addr 127.0.0.1 --master-port 29558 bench.py --gpus 1 --force-slab --halo fused --steps 5 --warmup 3 --no-e2e --no-cpu 2>/dev/null | grep '^{' | tail -1)
  echo "PDL=$e $(echo $r | python -c 'import json,sys; d=json.loads(sys.stdin.read()); print(round(d["value"],1))')"
done
