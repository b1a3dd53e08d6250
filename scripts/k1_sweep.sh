#!/bin/bash
# tuning sweep: K1 tile variants x L2 promotion, on the Gaussian, J3D7 promo only
one() { timeout 300 python bench.py --workload $1 --no-cpu --no-e2e --steps ${2:-20} 2>&1 | tail -1 | python -c "
import json,sys; d=json.loads(sys.stdin.read()); print('$1 K1V='\$LIFT_K1_VARIANT' PROMO='\$LIFT_L2PROMO, round(d['value'],1), 'Gpts/s', round(d['roofline']['achieved']), 'GB/s', round(d['roofline']['frac'],3))"; }
export LIFT_L2PROMO=3
for v in 0 1 2 4 5; do export LIFT_K1_VARIANT=$v; one gauss5_8192_mirror; done
export LIFT_K1_VARIANT=0
for pr in 0 1 2; do export LIFT_L2PROMO=$pr; one gauss5_8192_mirror; one j3d7_512_clamp 5; done
