mkdir -p gpurun_out/flush
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/flush/pytest_gpu.log 2>&1; tail -1 gpurun_out/flush/pytest_gpu.log
for w in c1 c2; do
  timeout 200 python bench.py --workload $w --no-e2e --no-cpu --steps 50 > gpurun_out/flush/${w}.json 2>&1
  echo $w $(python -c "import json,sys;d=json.loads(open('gpurun_out/flush/${w}.json').read().strip().splitlines()[-1]);print(d['ms_per_step'],d['roofline']['kernel_ms'],d['roofline']['frac'])")
done
timeout 300 python bench.py --no-e2e --no-cpu > gpurun_out/flush/c4.json 2>&1
echo c4 $(python -c "import json,sys;d=json.loads(open('gpurun_out/flush/c4.json').read().strip().splitlines()[-1]);print(d['ms_per_step'],d['roofline']['kernel_ms'],d['roofline']['frac'])")
timeout 300 ncu --metrics gpu__time_duration.sum --clock-control none --csv python bench.py --workload c1 --steps 2 --warmup 3 --no-e2e --no-cpu > gpurun_out/flush/c1_launches.csv 2>/dev/null
