mkdir -p gpurun_out/c1ncu
for w in c1 c2; do
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,sm__cycles_active.avg,launch__grid_size --clock-control none --csv python bench.py --workload $w --steps 2 --warmup 3 --no-e2e --no-cpu > gpurun_out/c1ncu/${w}_launches.csv 2>/dev/null
done
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_sga_bulk -s 3 -c 1 -o gpurun_out/c1ncu/c1_bulk_full python bench.py --workload c1 --steps 2 --warmup 3 --no-e2e --no-cpu > /dev/null 2>&1
ls gpurun_out/c1ncu
