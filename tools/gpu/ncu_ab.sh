# ncu of the C4 kernel for the current build and build/ab/*.so
TAG=${TAG:-ncuab}
mkdir -p gpurun_out/$TAG
one() {  # name, lib
  OCL_LIB_PATH=$2 AB_STEPS=1 timeout 600 ncu --set full --import-source on --clock-control none -k regex:k_sga_bulk -s 3 -c 1 \
    -o gpurun_out/$TAG/$1 -f python tools/dev/ab.py ${SPEC:-c4} > gpurun_out/$TAG/$1.log 2>&1
  ncu -i gpurun_out/$TAG/$1.ncu-rep --page details --csv > gpurun_out/$TAG/$1_details.csv 2>/dev/null
  ncu -i gpurun_out/$TAG/$1.ncu-rep --page raw --csv > gpurun_out/$TAG/$1_raw.csv 2>/dev/null
  ncu -i gpurun_out/$TAG/$1.ncu-rep --page source --csv --print-source sass > gpurun_out/$TAG/$1_sass.csv 2>/dev/null
  gzip -f gpurun_out/$TAG/$1_sass.csv; rm -f gpurun_out/$TAG/$1.ncu-rep
}
one new $PWD/paper_journals_pvldb_heimelspmm13_b200/_lib/libocelot_b200.so
for so in build/ab/*.so; do one $(basename $so .so) $PWD/$so; done
SPECS="${SPEC:-c4}" bash tools/gpu/ab.sh > /dev/null 2>&1; cp gpurun_out/ab/ab.txt gpurun_out/$TAG/ 2>/dev/null
ls gpurun_out/$TAG
