TAG=${TAG:-abjit}
mkdir -p gpurun_out/$TAG
timeout 600 python tools/dev/ab.py ${SPECS} | sed "s/^/aot /" >> gpurun_out/$TAG/ab.txt 2>&1
OCL_JIT_ALL=1 timeout 600 python tools/dev/ab.py ${SPECS} | sed "s/^/jit /" >> gpurun_out/$TAG/ab.txt 2>&1
cat gpurun_out/$TAG/ab.txt
