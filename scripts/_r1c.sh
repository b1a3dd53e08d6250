mkdir -p gpurun_out
timeout 600 python -m pytest tests -m gpu -x -q -k "srad" 2>&1 | tail -3
python scripts/tune_sweep.py srad_iter_4096:10: srad_iter_4096:10:LIFT_SRAD_SHAPE=1 srad_iter_4096:10:LIFT_SRAD_SHAPE=2 srad_iter_4096:10:LIFT_SRAD_SHAPE=3 srad_iter_4096:10:LIFT_SRAD_SHAPE=4 2>&1 | tee gpurun_out/sweep_srad.txt
bash scripts/ncu_full.sh r1c "t1_poisson19_512:k2_sweep" "t1_jacobi3d13_512:k2_sweep" "srad_iter_4096:k1_srad_fused" > /dev/null 2>&1
for w in t1_poisson19_512 t1_jacobi3d13_512 srad_iter_4096; do python scripts/stall_top.py gpurun_out/ncu_r1c_$w.ncu-rep 30 > gpurun_out/stall_r1c_$w.txt 2>&1; done
ls gpurun_out
