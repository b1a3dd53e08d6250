#!/bin/bash
# K2R integration pass (under gpurun): GPU suite, default bench line, 3D weighted
# workloads, ncu launch list of the default bench command, DRAM bytes of K2R.
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -4 > gpurun_out/r02k_pytest.txt
timeout 600 python bench.py > gpurun_out/r02k_bench.json 2> gpurun_out/r02k_bench.err
timeout 600 python bench.py --time-block 1 --no-cpu > gpurun_out/r02k_bench_tb1.json 2> /dev/null
timeout 900 python scripts/tune_sweep.py j3d7_512_clamp:10: t1_heat7_512:10: t1_jacobi3d7_256:10: > gpurun_out/r02k_sweep.txt 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv \
  --log-file gpurun_out/r02k_ncu_launches_j3d7.csv python bench.py --steps 2 --warmup 3 --no-cpu --no-e2e > /dev/null 2>&1
timeout 900 python scripts/ncu_bytes.py j3d7_512_clamp t1_heat7_512 t1_jacobi3d7_256 > gpurun_out/r02k_ncu_bytes.log 2>&1
echo done
