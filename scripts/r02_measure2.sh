#!/bin/bash
# Round-2 final measurement pass (under gpurun): GPU suite, default bench line
# (two-step K2R), --time-block 1 line, reference arm, every workload, the ncu
# launch list of the default bench command, ncu --set full of its top kernel,
# DRAM bytes per point of every config (incl. the two-step kernels).
mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -q 2>&1 | tail -3 > gpurun_out/m2_pytest.txt
timeout 600 python bench.py > gpurun_out/m2_bench_default.json 2> gpurun_out/m2_bench_default.err
timeout 600 python bench.py --time-block 1 > gpurun_out/m2_bench_tb1.json 2> /dev/null
timeout 600 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/m2_bench_reference.json 2>&1
timeout 2400 python scripts/tune_sweep.py $(python -c "import stencil_inputs as s; print(' '.join(w + ':10:' for w in s.WORKLOAD_NAMES))") \
  > gpurun_out/m2_sweep_all.txt 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv \
  --log-file gpurun_out/m2_ncu_launches_j3d7.csv python bench.py --steps 2 --warmup 3 --no-cpu --no-e2e > gpurun_out/m2_ncu_launches_bench.log 2>&1
bash scripts/ncu_full.sh m2 "j3d7_512_clamp:k2r" > /dev/null 2>&1
timeout 2400 python scripts/ncu_bytes.py > gpurun_out/m2_ncu_bytes.log 2>&1
echo done
