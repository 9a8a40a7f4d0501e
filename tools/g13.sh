cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python tools/order_probe.py > gpurun_out/g13_order.json 2>&1
timeout 300 python tools/mandel_probe.py > gpurun_out/g13_mandel.json 2>&1
timeout 900 python tools/lmosem_scaling_proxy.py > gpurun_out/g13_proxy.jsonl 2>&1
timeout 900 python -m pytest tests/test_gpu_lmosem.py tests/test_gpu_graphs.py -m gpu -q -x > gpurun_out/g13_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g13_pytest.log
tail -3 gpurun_out/g13_pytest.log; cat gpurun_out/g13_order.json gpurun_out/g13_mandel.json gpurun_out/g13_proxy.jsonl
