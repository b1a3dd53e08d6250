#!/bin/bash
# ncu --set full of one K2R launch per shape (under gpurun).  usage: bash scripts/ncu_k2r.sh TAG RPW...
TAG=$1; shift
mkdir -p gpurun_out
for r in "$@"; do
  LIFT_K2R_SHAPE=$r timeout 600 ncu --set full --clock-control none --import-source on -k "regex:k2r" --launch-skip 3 --launch-count 1 \
    -o gpurun_out/ncu_${TAG}_k2r_$r -f python scripts/k2r_once.py > gpurun_out/ncu_${TAG}_k2r_$r.log 2>&1
  python scripts/ncu_summary.py gpurun_out/ncu_${TAG}_k2r_$r.ncu-rep > gpurun_out/ncu_${TAG}_k2r_$r.txt 2>&1
done
