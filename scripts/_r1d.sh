mkdir -p gpurun_out
timeout 600 python -m pytest tests -m gpu -x -q -k "box or poisson or bitwise or srad" 2>&1 | tail -3
python scripts/tune_sweep.py t1_poisson19_512:10: t1_poisson19_512:10:LIFT_K2_BOX=1 t1_poisson19_512:10:LIFT_K2_BOX=2 \
  t1_jacobi3d13_512:10: t1_jacobi3d13_512:10:LIFT_K2_R2=1 t1_jacobi3d13_512:10:LIFT_K2_R2=2 \
  acoustic13_1024:3: 2>&1 | tee gpurun_out/sweep_r1d.txt
