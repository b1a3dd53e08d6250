#!/bin/bash
# One gpurun pass: GPU parity tests, bench lines, ncu launch list + full capture of the top kernel.
# usage (under gpurun): bash scripts/gpu_check.sh [tag] [workload...]
TAG=${1:-run}; shift
WLS=${@:-j3d7_512_clamp}
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -15
for w in $WLS; do
  timeout 600 python bench.py --workload $w --no-cpu 2>&1 | tail -1 | tee gpurun_out/bench_${TAG}_${w}.json
done
