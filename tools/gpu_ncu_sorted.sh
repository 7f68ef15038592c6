mkdir -p gpurun_out/sorted
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sorted_agg -s 1 -c 1 -o gpurun_out/sorted/agg_full -f python bench.py --workload c3c --steps 1 --warmup 1 --no-e2e --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_sorted_summary -s 1 -c 1 -o gpurun_out/sorted/sum_full -f python bench.py --workload c3c --steps 1 --warmup 1 --no-e2e --no-cpu > /dev/null 2>&1
ls -la gpurun_out/sorted
