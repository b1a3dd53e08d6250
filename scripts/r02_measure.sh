#!/bin/bash
# Round-2 measurement pass (under gpurun): default bench line, reference arm,
# every workload, the ncu launch list of the default bench command, ncu
# --set full of its top kernel, DRAM bytes per point of every config.
mkdir -p gpurun_out
timeout 600 python bench.py > gpurun_out/r02_bench_default.json 2> gpurun_out/r02_bench_default.err
tail -c 1500 gpurun_out/r02_bench_default.json
timeout 600 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/r02_bench_reference.json 2>&1
timeout 1800 python scripts/tune_sweep.py $(python -c "import stencil_inputs as s; print(' '.join(w + ':10:' for w in s.WORKLOAD_NAMES))") \
  > gpurun_out/r02_sweep_all.txt 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv \
  --log-file gpurun_out/r02_ncu_launches_j3d7.csv python bench.py --steps 2 --warmup 3 --no-cpu --no-e2e > gpurun_out/r02_ncu_launches_bench.log 2>&1
bash scripts/ncu_full.sh r02 "j3d7_512_clamp:k2_sweep" > /dev/null 2>&1
timeout 1800 python scripts/ncu_bytes.py > gpurun_out/r02_ncu_bytes.log 2>&1
echo done
