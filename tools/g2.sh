cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_lmosem.py tests/test_gpu_coherence.py -m gpu -q -x > gpurun_out/g2_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g2_pytest.log
timeout 900 python tools/lm_lanes_probe.py > gpurun_out/g2_lanes.jsonl 2> gpurun_out/g2_lanes.err
LM_MINB=4 LM_BLOCKS=256 LM_ORDER=x timeout 600 python tools/lm_lanes_probe.py > gpurun_out/g2_lanes_minb4.jsonl 2>> gpurun_out/g2_lanes.err
tail -3 gpurun_out/g2_pytest.log; cat gpurun_out/g2_lanes.jsonl
