#!/bin/bash
# ncu --set full of one fused slab step (world size 1, torchrun)
mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on -k "regex:k2_sweep" --launch-skip 150 --launch-count 1 \
  -o gpurun_out/ncu_r02_fused -f python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 --master-addr 127.0.0.1 \
  --master-port 29557 bench.py --gpus 1 --force-slab --halo fused --steps 1 --warmup 3 --no-e2e --no-cpu > gpurun_out/ncu_r02_fused.log 2>&1
python scripts/ncu_summary.py gpurun_out/ncu_r02_fused.ncu-rep > gpurun_out/ncu_r02_fused.txt 2>&1
python scripts/stall_top.py gpurun_out/ncu_r02_fused.ncu-rep 20 >> gpurun_out/ncu_r02_fused.txt 2>&1
cat gpurun_out/ncu_r02_fused.txt | head -45
