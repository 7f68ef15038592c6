# ncu --set full captures of the signature kernels (one launch each) + source hot spots
TAG=${TAG:-ncu}
mkdir -p gpurun_out/$TAG
cap() {  # name, bench args
  timeout 600 ncu --set full --import-source on --clock-control none -k regex:k_sga_bulk -s 2 -c 1 -o gpurun_out/$TAG/$1 -f \
    python bench.py --no-cpu --no-e2e --steps 1 --warmup 2 $2 > gpurun_out/$TAG/$1.log 2>&1
  ncu -i gpurun_out/$TAG/$1.ncu-rep --page raw --csv > gpurun_out/$TAG/$1_raw.csv 2>/dev/null
  ncu -i gpurun_out/$TAG/$1.ncu-rep --page source --csv --print-source sass > gpurun_out/$TAG/$1_sass.csv 2>/dev/null
  ncu -i gpurun_out/$TAG/$1.ncu-rep --page details --csv > gpurun_out/$TAG/$1_details.csv 2>/dev/null
  gzip -f gpurun_out/$TAG/$1_sass.csv; [ -n "$KEEP" ] || rm -f gpurun_out/$TAG/$1.ncu-rep
}
cap c5_g16 "--workload c5 --c5-groups 16"
cap c5_g256 "--workload c5 --c5-groups 256"
cap c4 "--workload c4"
ls -la gpurun_out/$TAG
