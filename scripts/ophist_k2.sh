#!/bin/bash
# ncu op histograms of the K2 sweeps (J3D7, J3D13, Acoustic-13)
for wl in j3d7_512_clamp t1_jacobi3d13_512 acoustic13_1024; do
  bash scripts/ncu_full.sh r02oh "$wl:k2_sweep" > /dev/null 2>&1
  echo "== $wl"; python scripts/op_hist.py gpurun_out/ncu_r02oh_$wl.ncu-rep | head -24
done
