TAG=${TAG:-absparse}
mkdir -p gpurun_out/$TAG
S="c5:4:0:0.01 c5:4:0:0.5 c5:4:0:1.0 c5:256:0:0.01 c5:256:0:0.5 c5:256:0:1.0 c5:1024:1.0:0.01 c5:16:1.5:0.01"
timeout 600 python tools/dev/ab.py $S | sed "s/^/dense  /" >> gpurun_out/$TAG/ab.txt 2>&1
OCL_SPARSE=1 timeout 600 python tools/dev/ab.py $S | sed "s/^/sparse /" >> gpurun_out/$TAG/ab.txt 2>&1
cat gpurun_out/$TAG/ab.txt
