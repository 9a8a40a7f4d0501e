cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_scan_progress.py tests/test_gpu_graphs.py tests/test_gpu_skeletons.py tests/test_gpu_distributions.py tests/test_gpu_fullsize.py tests/test_gpu_small_paths.py -m gpu -q -x > gpurun_out/g1_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g1_pytest.log
timeout 600 python bench.py > gpurun_out/g1_bench.json 2> gpurun_out/g1_bench.err
tail -5 gpurun_out/g1_pytest.log
