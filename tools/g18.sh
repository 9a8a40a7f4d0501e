cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_mandelbrot.py -m gpu -q -x -k "refill or tiles_periodic" > gpurun_out/g18_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g18_pytest.log
timeout 300 python tools/mandel_probe.py > gpurun_out/g18_mandel.jsonl 2>&1
MANDEL_THREADS=$((148*2048)) timeout 300 python tools/mandel_probe.py >> gpurun_out/g18_mandel.jsonl 2>&1
MANDEL_THREADS=$((148*512)) timeout 300 python tools/mandel_probe.py >> gpurun_out/g18_mandel.jsonl 2>&1
SKEL_NVRTC_DEFINES="-DMANDEL_CHUNK=64" timeout 300 python tools/mandel_probe.py >> gpurun_out/g18_mandel.jsonl 2>&1
tail -3 gpurun_out/g18_pytest.log; cat gpurun_out/g18_mandel.jsonl
