cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_mandelbrot.py -m gpu -q -x -k "periodic" > gpurun_out/g8_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g8_pytest.log
for d in "" "-DMANDEL_B=16"; do SKEL_NVRTC_DEFINES="$d" timeout 300 python tools/mandel_probe.py >> gpurun_out/g8_mandel.jsonl 2>&1; done
tail -3 gpurun_out/g8_pytest.log; cat gpurun_out/g8_mandel.jsonl
