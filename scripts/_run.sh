cd $GRAFT_REPO_ROOT
for d in _old .; do
 for i in 1 2; do
  (cd $d && timeout 300 python bench.py --workload hotspot3d_8x512x512 --no-cpu --no-e2e --steps 20 2>&1 | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('$d', round(d['value'],1), d['roofline']['avg_launch_us'])")
  (cd $d && timeout 300 python bench.py --workload hotspot3d_8x512x512 --no-cpu --no-e2e --no-graph --steps 20 2>&1 | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('$d nograph', round(d['value'],1), d['roofline']['avg_launch_us'])")
 done
done
