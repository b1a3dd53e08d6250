#!/bin/bash
# compute-sanitizer over K2R (two-step register kernel): small tile/chunk/boundary cases
mkdir -p gpurun_out
K="test_k2r_bitwise and (shape0-0 or shape3-kind2 or shape5-1 or shape9-kind3) or test_k2r_shapes_and_chunks and (zc0-4 or zc2-6) or odd_steps"
for tool in memcheck racecheck synccheck; do
  echo "== $tool"
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 --error-exitcode 9 \
     python -m pytest tests/test_tblock_gpu.py -q -x -k "$K" 2>&1 | tail -4
  echo "rc=${PIPESTATUS[0]}"
done
