# Round evidence: GPU test suite, smoke, bench lines (default C4 + reference arm + other configs), launch lists.
set -x
mkdir -p gpurun_out/round
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/round/pytest_gpu.log 2>&1; tail -3 gpurun_out/round/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/round/smoke.log 2>&1; tail -1 gpurun_out/round/smoke.log
timeout 400 python bench.py > gpurun_out/round/bench_c4.json 2> gpurun_out/round/bench_c4.err
timeout 400 python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/round/bench_ref.json 2>&1
for w in c1 c2 c3 c3c j3; do timeout 300 python bench.py --workload $w --no-e2e > gpurun_out/round/bench_$w.json 2>&1; done
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu > gpurun_out/round/c4_launches.csv 2>/dev/null
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload c3c --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/round/c3c_launches.csv 2>/dev/null
ls -la gpurun_out/round
