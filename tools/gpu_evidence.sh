mkdir -p gpurun_out/ev
timeout 400 python bench.py > gpurun_out/ev/bench_c4.json 2> gpurun_out/ev/bench_c4.err; tail -c 300 gpurun_out/ev/bench_c4.json
for w in c1 c2 c3; do timeout 300 python bench.py --workload $w --no-e2e > gpurun_out/ev/bench_$w.json 2>&1; done
for w in c1 c2 c4; do
timeout 400 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload $w --steps 2 --warmup 3 --no-e2e --no-cpu > gpurun_out/ev/${w}_launches.csv 2>/dev/null
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sga_bulk -s 3 -c 1 -o gpurun_out/ev/c4_k_sga_bulk_full python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu > /dev/null 2>&1
ls gpurun_out/ev
