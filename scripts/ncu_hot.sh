#!/bin/bash
# ncu --set full of one launch WITHOUT cache control (L2-warm, as in the
# back-to-back x100 graph): bash scripts/ncu_hot.sh TAG workload kernel_regex [env...]
TAG=$1; wl=$2; kr=$3; shift 3
mkdir -p gpurun_out
env "$@" timeout 600 ncu --set full --cache-control none --clock-control none --import-source on -k "regex:$kr" --launch-skip ${SKIP:-20} --launch-count 1 \
  -o gpurun_out/ncu_${TAG}_${wl} -f python bench.py --workload $wl --no-cpu --no-e2e --no-graph --no-flush --steps 1 --warmup 3 > gpurun_out/ncu_${TAG}_${wl}.log 2>&1
python scripts/ncu_summary.py gpurun_out/ncu_${TAG}_${wl}.ncu-rep > gpurun_out/ncu_${TAG}_${wl}.txt 2>&1
ncu -i gpurun_out/ncu_${TAG}_${wl}.ncu-rep --page details > gpurun_out/ncu_${TAG}_${wl}_details.txt 2>&1
python scripts/stall_top.py gpurun_out/ncu_${TAG}_${wl}.ncu-rep 20 >> gpurun_out/ncu_${TAG}_${wl}.txt 2>&1
grep -E "Duration|Elapsed Cycles|SM Active Cycles|Memory Throughput|DRAM Throughput|L2 Hit" gpurun_out/ncu_${TAG}_${wl}_details.txt | head -8
cat gpurun_out/ncu_${TAG}_${wl}.txt | head -40
