mkdir -p gpurun_out/radix
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_rs_scatter -s 1 -c 1 -o gpurun_out/radix/scatter_full -f python bench.py --workload c3 --tier 6 --steps 1 --warmup 0 --no-e2e --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_rs_hist -s 1 -c 1 -o gpurun_out/radix/hist_full -f python bench.py --workload c3 --tier 6 --steps 1 --warmup 0 --no-e2e --no-cpu > /dev/null 2>&1
ls -la gpurun_out/radix
