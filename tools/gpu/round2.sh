# Round-2 evidence: bench lines, launch lists, full ncu of the headline kernels, the C5 sweep, operators.
TAG=${TAG:-round2}
O=gpurun_out/$TAG
mkdir -p $O
nvidia-smi --query-gpu=name,clocks.max.sm,memory.total --format=csv > $O/gpu.txt 2>&1
b() { n=$1; shift; timeout 600 python bench.py "$@" > $O/bench_$n.json 2> $O/bench_$n.err; tail -c 300 $O/bench_$n.json; echo; }
b c4
b c4_dist --dist --no-cpu
b reference --impl reference --steps 3 --warmup 1
b c4mm --workload c4mm --no-e2e --no-cpu
b c2 --workload c2 --no-e2e
b c1 --workload c1 --no-e2e
b c1_graph --workload c1 --graph --no-e2e --no-cpu
b c3 --workload c3 --no-e2e
b c3c --workload c3c --no-e2e --no-cpu
b c3s --workload c3s --no-e2e --no-cpu
b j3 --workload j3 --no-cpu
for g in 4 16 256 1024 65536 16777216; do b c5_g$g --workload c5 --c5-groups $g --no-e2e --no-cpu; done
b c5_g256_sel1 --workload c5 --c5-groups 256 --c5-sel 0.01 --no-e2e --no-cpu
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_op_atom.sum,lts__t_sectors_op_red.sum,l1tex__data_pipe_lsu_wavefronts_mem_shared_op_atom.sum
l() { n=$1; shift; timeout 900 ncu --metrics $M --clock-control none --csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu "$@" > $O/${n}_launches.csv 2>/dev/null; }
l c4; l c4mm --workload c4mm; l c2 --workload c2; l c1 --workload c1; l c3 --workload c3; l c3c --workload c3c
for g in 16 256 1024 65536 16777216; do l c5_g$g --workload c5 --c5-groups $g; done
for f in $O/*_launches.csv; do python tools/launches.py $f 60 > ${f%.csv}.txt 2>&1; done
f() { n=$1; k=$2; shift 2; timeout 900 ncu --set full --import-source on --clock-control none -k regex:$k -s 1 -c 1 -o $O/$n -f python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu "$@" > /dev/null 2>&1
  ncu -i $O/$n.ncu-rep --page details --csv > $O/${n}_details.csv 2>/dev/null; ncu -i $O/$n.ncu-rep --page raw --csv > $O/${n}_raw.csv 2>/dev/null; rm -f $O/$n.ncu-rep; }
f c4_full k_sga_bulk; f c4mm_full k_sga_bulk --workload c4mm; f c5_g256_full k_sga_bulk --workload c5 --c5-groups 256; f c3_agg_full k_part_agg --workload c3; f c3_l1_full k_part_scatter_l1 --workload c3; f c3_s2_full k_part_scatter2 --workload c3
timeout 1800 python tools/sweep_c5.py --steps 5 --out $O/c5_sweep.json > $O/c5_sweep.log 2>&1
timeout 900 python tools/bench_ops.py --out $O/ops.json > $O/ops.log 2>&1
ls $O | wc -l
