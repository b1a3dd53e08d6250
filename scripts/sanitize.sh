#!/bin/bash
# compute-sanitizer passes over small parity cases (memcheck, racecheck, synccheck)
mkdir -p gpurun_out
K="kernel_families or degenerate or unaligned or mixed_kinds"
for tool in memcheck racecheck synccheck; do
  echo "== $tool"
  timeout 1200 compute-sanitizer --tool $tool --print-limit 20 --error-exitcode 9 \
     python -m pytest tests/test_parity_gpu.py -q -x -k "$K" 2>&1 | tail -8
  echo "rc=$?"
done
