mkdir -p gpurun_out/early
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/early/pytest_gpu.log 2>&1; tail -1 gpurun_out/early/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
for w in c1 c2 c4; do for rep in 1 2; do
  timeout 300 python bench.py --workload $w --no-e2e --no-cpu > gpurun_out/early/${w}_$rep.json 2>&1
  echo $w $(python -c "import json,sys;d=json.loads(open('gpurun_out/early/${w}_$rep.json').read().strip().splitlines()[-1]);print(d['ms_per_step'],d['roofline']['kernel_ms'],d['roofline']['frac'])")
done; done
