cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python tools/order_probe.py > gpurun_out/g6_order.json 2>&1
timeout 1500 python -m pytest tests/test_gpu_mandelbrot.py -m gpu -q -x -k cyclic > gpurun_out/g6_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g6_pytest.log
tail -3 gpurun_out/g6_pytest.log; cat gpurun_out/g6_order.json
