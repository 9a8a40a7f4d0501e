cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_mandelbrot.py tests/test_gpu_skeletons.py tests/test_gpu_graphs.py tests/test_gpu_lmosem.py -m gpu -q -x > gpurun_out/g5_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g5_pytest.log
timeout 300 python tools/mandel_probe.py > gpurun_out/g5_mandel.jsonl 2>&1
for d in "-DMANDEL_P=16" "-DMANDEL_PB=16" "-DMANDEL_P=4" "-DMANDEL_P=16 -DMANDEL_PB=16"; do SKEL_NVRTC_DEFINES="$d" timeout 300 python tools/mandel_probe.py >> gpurun_out/g5_mandel.jsonl 2>&1; done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv python tools/workload_once.py lmosem_device > gpurun_out/g5_order_launches.csv 2> gpurun_out/g5_ncu.err
tail -3 gpurun_out/g5_pytest.log; cat gpurun_out/g5_mandel.jsonl
