# GPU test files given in $FILES (default: all GPU tests), plus smoke
TAG=${TAG:-verify}
mkdir -p gpurun_out/$TAG
timeout ${PYT_TIMEOUT:-2400} python -m pytest -q ${FILES:-tests} -m gpu > gpurun_out/$TAG/pytest.log 2>&1
tail -15 gpurun_out/$TAG/pytest.log | grep -E "passed|failed|FAILED|Error" | head -20
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
