# ncu --set full of one unfused operator kernel (regex $K) in tools/bench_ops.py --only $ONLY
TAG=${TAG:-ncuops}
mkdir -p gpurun_out/$TAG
name=${NAME:-op}
timeout 900 ncu --set full --import-source on --clock-control none -k regex:$K -s ${SKIP:-2} -c 1 -o gpurun_out/$TAG/$name -f \
  python tools/bench_ops.py --only $ONLY --steps 1 --warmup 1 --rows ${ROWS:-200000000} > gpurun_out/$TAG/$name.log 2>&1
ncu -i gpurun_out/$TAG/$name.ncu-rep --page raw --csv > gpurun_out/$TAG/${name}_raw.csv 2>/dev/null
ncu -i gpurun_out/$TAG/$name.ncu-rep --page source --csv --print-source sass > gpurun_out/$TAG/${name}_sass.csv 2>/dev/null
gzip -f gpurun_out/$TAG/${name}_sass.csv; rm -f gpurun_out/$TAG/$name.ncu-rep
