mkdir -p gpurun_out/c1f
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_sga_bulk -s 3 -c 1 -o gpurun_out/c1f/c1_bulk_full python bench.py --workload c1 --steps 2 --warmup 3 --no-e2e --no-cpu > /dev/null 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_sga_bulk -s 3 -c 1 -o gpurun_out/c1f/c2_bulk_full python bench.py --workload c2 --steps 2 --warmup 3 --no-e2e --no-cpu > /dev/null 2>&1
ls gpurun_out/c1f
