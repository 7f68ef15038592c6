TAG=${TAG:-repro}
mkdir -p gpurun_out/$TAG
timeout 600 python tools/dev/repro_bulk.py 909329 8 > gpurun_out/$TAG/repro.log 2>&1
timeout 300 python tools/dev/repro_bulk.py 2000000 4 4,3 >> gpurun_out/$TAG/repro.log 2>&1
cat gpurun_out/$TAG/repro.log | grep -v "^  " 
timeout 400 python bench.py --no-cpu --no-e2e > gpurun_out/$TAG/bench_c4.json 2>&1; tail -c 400 gpurun_out/$TAG/bench_c4.json
timeout 400 python bench.py --no-cpu --no-e2e --workload c2 > gpurun_out/$TAG/bench_c2.json 2>&1; tail -c 300 gpurun_out/$TAG/bench_c2.json
timeout 400 python bench.py --no-cpu --no-e2e --workload c1 > gpurun_out/$TAG/bench_c1.json 2>&1; tail -c 300 gpurun_out/$TAG/bench_c1.json
