# Round evidence: bench lines, reference arm, launch list, full ncu capture, C5 sweep.
set -x
mkdir -p gpurun_out/round
timeout 400 python bench.py > gpurun_out/round/bench_c4.json 2> gpurun_out/round/bench_c4.err
timeout 400 python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/round/bench_ref.json 2>&1
for w in c1 c2 c3 c3c; do timeout 300 python bench.py --workload $w --no-e2e > gpurun_out/round/bench_$w.json 2>&1; done
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu > gpurun_out/round/c4_launches.csv 2>/dev/null
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sga_bulk -s 1 -c 1 -o gpurun_out/round/c4_k_sga_bulk_full -f python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu > /dev/null 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload c3 --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/round/c3_launches.csv 2>/dev/null
timeout 900 python tools/sweep_c5.py --steps 5 --out gpurun_out/round/c5_sweep.json > gpurun_out/round/c5_sweep.log 2>&1
