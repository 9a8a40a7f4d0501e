cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_fused.py -m gpu -q -x -rs -k multicast > gpurun_out/g11_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g11_pytest.log
tail -8 gpurun_out/g11_pytest.log
