cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_lmosem.py -m gpu -q -x -k "device or lanes" > gpurun_out/g4_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g4_pytest.log
timeout 900 python tools/lmosem_scaling_proxy.py > gpurun_out/g4_proxy.jsonl 2> gpurun_out/g4_proxy.err
timeout 900 ncu --kernel-name skel_ew_kernel --launch-skip 7 --launch-count 1 --set full --import-source on -o gpurun_out/g4_mandel_paper -f python tools/mandel_probe.py > gpurun_out/g4_ncu1.log 2>&1
timeout 900 ncu --kernel-name skel_ew_kernel --launch-skip 24 --launch-count 1 --set full --import-source on -o gpurun_out/g4_mandel_blocked -f python tools/mandel_probe.py > gpurun_out/g4_ncu2.log 2>&1
timeout 300 python tools/mandel_probe.py > gpurun_out/g4_mandel.json 2>&1
tail -3 gpurun_out/g4_pytest.log; cat gpurun_out/g4_proxy.jsonl; cat gpurun_out/g4_mandel.json; tail -3 gpurun_out/g4_ncu1.log
