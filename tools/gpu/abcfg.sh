TAG=${TAG:-abcfg}
mkdir -p gpurun_out/$TAG
for c in 7 3 2 6 5 1; do OCL_BULK=$c timeout 600 python tools/dev/ab.py ${SPECS:-c4mm} | sed "s/^/cfg$c /" >> gpurun_out/$TAG/ab.txt 2>&1; done
cat gpurun_out/$TAG/ab.txt
