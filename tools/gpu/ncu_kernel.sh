# ncu --set full of one kernel (regex $K) in a bench run ($ARGS); summaries only
TAG=${TAG:-ncuk}
mkdir -p gpurun_out/$TAG
name=${NAME:-k}
timeout 900 ncu --set full --import-source on --clock-control none -k regex:$K -s ${SKIP:-1} -c 1 -o gpurun_out/$TAG/$name -f \
  python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu $ARGS > gpurun_out/$TAG/$name.log 2>&1
ncu -i gpurun_out/$TAG/$name.ncu-rep --page details --csv > gpurun_out/$TAG/${name}_details.csv 2>/dev/null
ncu -i gpurun_out/$TAG/$name.ncu-rep --page raw --csv > gpurun_out/$TAG/${name}_raw.csv 2>/dev/null
ncu -i gpurun_out/$TAG/$name.ncu-rep --page source --csv --print-source sass > gpurun_out/$TAG/${name}_sass.csv 2>/dev/null
gzip -f gpurun_out/$TAG/${name}_sass.csv; [ -n "$KEEP" ] || rm -f gpurun_out/$TAG/$name.ncu-rep
ls gpurun_out/$TAG
