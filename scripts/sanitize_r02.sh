#!/bin/bash
# compute-sanitizer over the round-2 kernels: K2C (few-plane column tiles),
# K6 (resident iterate), the K1S WRAP fix, the per-launch counter slots and
# bounded waits (small cases)
mkdir -p gpurun_out
K="column3d and (shape0 or shape1 or shape2) or resident3d and (shape1 or shape2) or srad_iteration"
for tool in memcheck racecheck synccheck; do
  echo "== $tool"
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 --error-exitcode 9 \
     python -m pytest tests/test_parity_gpu.py -q -x -k "$K" 2>&1 | tail -4
  echo "rc=${PIPESTATUS[0]}"
done
echo "== memcheck robust"
timeout 1500 compute-sanitizer --tool memcheck --print-limit 20 --error-exitcode 9 \
   python -m pytest tests/test_robust_gpu.py -q -x -k "dead or eager" 2>&1 | tail -4
