cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_rank_mode.py tests/test_gpu_lmosem.py -m gpu -q -x > gpurun_out/g14_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g14_pytest.log
timeout 300 python tools/order_probe.py > gpurun_out/g14_order.json 2>&1
tail -3 gpurun_out/g14_pytest.log; cat gpurun_out/g14_order.json
