cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
nvidia-smi -q | grep -i -A2 "fabric\|multicast" > gpurun_out/g9_smi.txt 2>&1
timeout 2400 python -m pytest tests/test_gpu_fused.py tests/test_gpu_vmm.py -m gpu -q -x -rs > gpurun_out/g9_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g9_pytest.log
tail -5 gpurun_out/g9_pytest.log; cat gpurun_out/g9_smi.txt | head -20
