TAG=${TAG:-sanitize}
mkdir -p gpurun_out/$TAG
timeout 2400 make sanitize > gpurun_out/$TAG/make.log 2>&1
cp profiles/sanitize_*.log gpurun_out/$TAG/ 2>/dev/null
cat gpurun_out/$TAG/make.log | tail -20
