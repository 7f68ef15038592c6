# A/B of an env switch ($ENVV) on the current build
TAG=${TAG:-abenv}
mkdir -p gpurun_out/$TAG
for r in 1 2; do
timeout 600 python tools/dev/ab.py ${SPECS} | sed "s/^/base /" >> gpurun_out/$TAG/ab.txt 2>&1
env $ENVV timeout 600 python tools/dev/ab.py ${SPECS} | sed "s/^/$ENVV /" >> gpurun_out/$TAG/ab.txt 2>&1
done
cat gpurun_out/$TAG/ab.txt
