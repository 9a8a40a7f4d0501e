cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 2400 python -m pytest tests/test_gpu_fused.py tests/test_gpu_vmm.py -m gpu -q -x -rs > gpurun_out/g10_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g10_pytest.log
tail -8 gpurun_out/g10_pytest.log
