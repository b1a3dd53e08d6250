#!/bin/bash
# K2R z-chunk pairs (long zc, tail zc2) on J3D7 512^3 x100 (under gpurun)
timeout 300 python scripts/k2r_probe.py 106:: 106:128:16 106:112:16 106:64:16 106:48:8 106:64:8 106:96:16 106:160:0 106:25:4 2>&1
