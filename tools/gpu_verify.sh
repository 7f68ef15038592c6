mkdir -p gpurun_out/verify
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/verify/pytest_gpu.log 2>&1; tail -1 gpurun_out/verify/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 400 python bench.py > gpurun_out/verify/bench_c4.json 2> gpurun_out/verify/bench_c4.err; tail -c 400 gpurun_out/verify/bench_c4.json
timeout 400 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/verify/bench_reference.json 2>&1; tail -c 200 gpurun_out/verify/bench_reference.json
for w in c2 c3; do timeout 300 python bench.py --workload $w --no-e2e > gpurun_out/verify/bench_$w.json 2>&1; done
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu > gpurun_out/verify/c4_launches.csv 2>/dev/null
ls gpurun_out/verify
