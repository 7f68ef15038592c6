mkdir -p gpurun_out/final
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/final/pytest_gpu.log 2>&1; tail -2 gpurun_out/final/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 400 python bench.py > gpurun_out/final/bench_c4.json 2> gpurun_out/final/bench_c4.err
for w in c3 j3; do timeout 300 python bench.py --workload $w --no-e2e > gpurun_out/final/bench_$w.json 2>&1; done
for w in j3; do timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload $w --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/final/${w}_launches.csv 2>/dev/null; done
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload c3 --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/final/c3_launches.csv 2>/dev/null
ls gpurun_out/final
