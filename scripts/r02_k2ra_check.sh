#!/bin/bash
# K2RA pass (under gpurun): tests, Acoustic bench lines (two-step default and
# --time-block 1), shapes, ncu of one K2RA launch per radius
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_tblock_gpu.py -x -q 2>&1 | tail -3 > gpurun_out/k2ra_tests.txt
for wl in acoustic7_1024 acoustic13_1024; do
  timeout 600 python bench.py --workload $wl --no-cpu > gpurun_out/k2ra_bench_$wl.json 2> /dev/null
  timeout 600 python bench.py --workload $wl --no-cpu --no-e2e --time-block 1 > gpurun_out/k2ra_bench_${wl}_tb1.json 2> /dev/null
done
for v in 4 8; do LIFT_K2RA_SHAPE=$v timeout 300 python bench.py --workload acoustic7_1024 --no-cpu --no-e2e --steps 5 2>/dev/null | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('a7 shape $v', d['value'])"; done >> gpurun_out/k2ra_shapes.txt
for v in 2 3; do LIFT_K2RA_SHAPE=$v timeout 300 python bench.py --workload acoustic13_1024 --no-cpu --no-e2e --steps 5 2>/dev/null | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('a13 shape $v', d['value'])"; done >> gpurun_out/k2ra_shapes.txt
bash scripts/ncu_full.sh k2ra "acoustic13_1024:k2ra" "acoustic7_1024:k2ra" > /dev/null 2>&1
echo done
