timeout 600 python bench.py --workload j3 --steps 10 > gpurun_out/j3.json 2> gpurun_out/j3.err; tail -c 1500 gpurun_out/j3.json; tail -3 gpurun_out/j3.err
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload j3 --steps 1 --warmup 1 --no-cpu > gpurun_out/j3_launches.csv 2>/dev/null
python tools/launches.py gpurun_out/j3_launches.csv 8
