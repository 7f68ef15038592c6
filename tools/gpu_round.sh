# Round evidence: GPU test suite, smoke, bench lines (default C4 + reference arm + other configs), launch lists, ncu.
set -x
mkdir -p gpurun_out/round
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/round/pytest_gpu.log 2>&1; tail -3 gpurun_out/round/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/round/smoke.log 2>&1; tail -1 gpurun_out/round/smoke.log
timeout 400 python bench.py > gpurun_out/round/bench_c4.json 2> gpurun_out/round/bench_c4.err
timeout 400 python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/round/bench_ref.json 2>&1
for w in c1 c2 c3 c3c c3s j3; do timeout 300 python bench.py --workload $w --no-e2e > gpurun_out/round/bench_$w.json 2>&1; done
timeout 300 python bench.py --workload c1 --graph --no-e2e > gpurun_out/round/bench_c1_graph.json 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu > gpurun_out/round/c4_launches.csv 2>/dev/null
for w in c3 c3c c3s j3; do timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload $w --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/round/${w}_launches.csv 2>/dev/null; done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_rs_scatter -s 1 -c 1 -o gpurun_out/round/c3s_k_rs_scatter_full -f python bench.py --workload c3s --steps 1 --warmup 0 --no-e2e --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_join_probe_pk -s 1 -c 1 -o gpurun_out/round/j3_k_join_probe_full -f python bench.py --workload j3 --steps 1 --warmup 1 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_part_agg -s 1 -c 1 -o gpurun_out/round/c3_k_part_agg_full -f python bench.py --workload c3 --steps 1 --warmup 0 --no-e2e --no-cpu > /dev/null 2>&1
timeout 1200 python tools/sweep_c5.py --steps 5 --out gpurun_out/round/c5_sweep.json > gpurun_out/round/c5_sweep.log 2>&1
ls -la gpurun_out/round
