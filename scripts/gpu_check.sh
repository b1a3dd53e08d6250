#!/bin/bash
# One gpurun pass: GPU parity tests, the default bench line, a sweep over every
# workload, the ncu launch list of the default bench command.
# usage (under gpurun): bash scripts/gpu_check.sh [tag]
TAG=${1:-run}
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -4 | tee gpurun_out/pytest_${TAG}.txt
timeout 600 python bench.py 2>&1 | tail -1 | tee gpurun_out/bench_${TAG}.json
timeout 1200 python scripts/tune_sweep.py $(python -c "import stencil_inputs as s; print(' '.join(w + ':10:' for w in s.WORKLOAD_NAMES))") \
  2>&1 | tee gpurun_out/sweep_${TAG}.txt
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv \
  --log-file gpurun_out/launches_${TAG}.csv python bench.py --steps 1 --warmup 3 --no-cpu --no-e2e > /dev/null 2>&1
echo done
