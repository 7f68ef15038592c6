# A/B of library builds: current tree vs build/ab/*.so on the same box
TAG=${TAG:-ab}
mkdir -p gpurun_out/$TAG
SPECS=${SPECS:-"c4 c2 c5:4 c5:16 c5:256"}
for r in 1 2; do
  timeout 600 python tools/dev/ab.py $SPECS >> gpurun_out/$TAG/ab.txt 2>&1
  for so in build/ab/*.so; do OCL_LIB_PATH=$PWD/$so timeout 600 python tools/dev/ab.py $SPECS >> gpurun_out/$TAG/ab.txt 2>&1; done
done
cat gpurun_out/$TAG/ab.txt
