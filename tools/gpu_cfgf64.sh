mkdir -p gpurun_out/f64
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/f64/pytest_gpu.log 2>&1; tail -1 gpurun_out/f64/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 300 python bench.py --workload c2 > gpurun_out/f64/bench_c2.json 2>&1
timeout 400 python bench.py > gpurun_out/f64/bench_c4.json 2>&1
for w in c2 c4; do echo $w $(python -c "import json,sys;d=json.loads(open('gpurun_out/f64/bench_$w.json').read().strip().splitlines()[-1]);print(d['ms_per_step'],d['roofline']['kernel_ms'],d['roofline']['frac'],d['roofline']['kernel'])"); done
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload c2 --steps 2 --warmup 3 --no-e2e --no-cpu > gpurun_out/f64/c2_launches.csv 2>/dev/null
