# ncu --set full of k_sga_bulk for the given ab.py specs (NAME=SPEC pairs); summaries only
TAG=${TAG:-ncuspec}
mkdir -p gpurun_out/$TAG
for pair in $PAIRS; do
  name=${pair%%=*}; spec=${pair#*=}
  AB_STEPS=1 timeout 600 ncu --set full --import-source on --clock-control none -k regex:k_sga_bulk -s 3 -c 1 \
    -o gpurun_out/$TAG/$name -f python tools/dev/ab.py $spec > gpurun_out/$TAG/$name.log 2>&1
  ncu -i gpurun_out/$TAG/$name.ncu-rep --page details --csv > gpurun_out/$TAG/${name}_details.csv 2>/dev/null
  ncu -i gpurun_out/$TAG/$name.ncu-rep --page raw --csv > gpurun_out/$TAG/${name}_raw.csv 2>/dev/null
  ncu -i gpurun_out/$TAG/$name.ncu-rep --page source --csv --print-source sass > gpurun_out/$TAG/${name}_sass.csv 2>/dev/null
  gzip -f gpurun_out/$TAG/${name}_sass.csv; [ -n "$KEEP" ] || rm -f gpurun_out/$TAG/$name.ncu-rep
done
ls gpurun_out/$TAG
