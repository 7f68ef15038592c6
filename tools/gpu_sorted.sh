# sorted-input GROUP BY: parity tests, C3 clustered bench (sorted vs hash), launch list
mkdir -p gpurun_out/sorted
summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', d['ms_per_step'], d['value']/1e9, d['roofline']['kernel'], d['roofline']['kernel_ms'])"; }
timeout 900 python -m pytest tests/test_gpu_sorted.py -x -q > gpurun_out/sorted/pytest.log 2>&1; echo "pytest rc=$?"; tail -30 gpurun_out/sorted/pytest.log
timeout 300 python bench.py --workload c3c --no-cpu --no-e2e --steps 20 > gpurun_out/sorted/c3c.json 2> gpurun_out/sorted/c3c.err; summ c3c-sorted < gpurun_out/sorted/c3c.json; tail -3 gpurun_out/sorted/c3c.err
timeout 300 python bench.py --workload c3c --no-sorted --no-cpu --no-e2e --steps 20 2>&1 | summ c3c-hash
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload c3c --steps 2 --warmup 1 --no-e2e --no-cpu > gpurun_out/sorted/c3c_launches.csv 2>/dev/null
python tools/launches.py gpurun_out/sorted/c3c_launches.csv 2>&1 | tail -15
