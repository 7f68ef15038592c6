# wait-mode A/B on the current build + the old build, same box
TAG=${TAG:-abw}
mkdir -p gpurun_out/$TAG
for r in 1 2; do
for w in 00 10; do OCL_WAIT=$w timeout 600 python tools/dev/ab.py ${SPECS:-c4 c2} | sed "s/^/W$w /" >> gpurun_out/$TAG/ab.txt 2>&1; done
for so in build/ab/*.so; do OCL_LIB_PATH=$PWD/$so timeout 600 python tools/dev/ab.py ${SPECS:-c4 c2} >> gpurun_out/$TAG/ab.txt 2>&1; done
done
cat gpurun_out/$TAG/ab.txt
