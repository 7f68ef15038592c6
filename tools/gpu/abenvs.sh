# A/B of several env settings (ENVS, separated by ';', "-" = none) x library builds (LIBS,
# space-separated .so paths, "-" = the current tree) on one box
TAG=${TAG:-abenvs}
LIBS=${LIBS:-"-"}
mkdir -p gpurun_out/$TAG
IFS=';' read -ra LIST <<< "$ENVS"
for r in 1 2; do
  for so in $LIBS; do
    lp=""; [ "$so" != "-" ] && lp="OCL_LIB_PATH=$PWD/$so"
    for e in "${LIST[@]}"; do
      lab="$(basename ${so/-/cur})|${e// /_}"
      [ "$e" = "-" ] && e=""
      env $lp $e timeout 600 python tools/dev/ab.py ${SPECS} | sed "s/^/$lab /" >> gpurun_out/$TAG/ab.txt 2>&1
    done
  done
done
awk '{print $1, $3, $4}' gpurun_out/$TAG/ab.txt | sort -k2,2 -k1,1
