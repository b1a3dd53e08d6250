#!/bin/bash
# ncu --set full capture of one launch of the dominant kernel per workload (under gpurun, one GPU).
# usage: bash scripts/ncu_full.sh TAG "workload:kernel_regex" ...
TAG=$1; shift
mkdir -p gpurun_out
for spec in "$@"; do
  wl=${spec%%:*}; kr=${spec#*:}
  timeout 600 ncu --set full --clock-control none --import-source on -k "regex:$kr" --launch-skip 3 --launch-count 1 \
    -o gpurun_out/ncu_${TAG}_${wl} -f python bench.py --workload $wl --no-cpu --no-e2e --no-graph --steps 1 --warmup 3 > gpurun_out/ncu_${TAG}_${wl}.log 2>&1
  python scripts/ncu_summary.py gpurun_out/ncu_${TAG}_${wl}.ncu-rep > gpurun_out/ncu_${TAG}_${wl}.txt 2>&1
  tail -30 gpurun_out/ncu_${TAG}_${wl}.txt
done
