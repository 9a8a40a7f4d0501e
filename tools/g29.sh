cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -x -q -k "reduce or scan or small or distrib or skeleton or fullsize" > gpurun_out/g29_pytest.log 2>&1; tail -3 gpurun_out/g29_pytest.log
echo "== new (one launch)"; timeout 600 python tools/small_n_probe.py 16 18 20 21 22 23 24
echo "== two launches"; SKEL_RED_SMALL_TWO=1 SKEL_SCAN_SMALL_TWO=1 timeout 600 python tools/small_n_probe.py 16 18 20 21 22 23 24
echo "== chain scan up to 2^25"; SKEL_SCAN_SMALL_MAX=33554432 timeout 600 python tools/small_n_probe.py 22 23 24 25
