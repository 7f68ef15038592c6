mkdir -p gpurun_out/c2cfg
for w in c2; do for c in 3 5 6 7 1 2; do
  OCL_BULK=$c timeout 200 python bench.py --workload $w --no-e2e --no-cpu --steps 50 > gpurun_out/c2cfg/${w}_$c.json 2>&1
  echo $w $c $(python -c "import json,sys;d=json.loads(open('gpurun_out/c2cfg/${w}_$c.json').read().strip().splitlines()[-1]);print(d['ms_per_step'],d['roofline']['kernel_ms'],d['roofline']['frac'])")
done; done
