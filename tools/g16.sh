cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_coherence.py tests/test_gpu_skeletons.py tests/test_gpu_distributions.py tests/test_gpu_rank_mode.py -m gpu -q -x > gpurun_out/g16_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g16_pytest.log
timeout 900 python bench.py --no-extras --no-cpu --e2e-steps 4 --steps 10 > gpurun_out/g16_bench.json 2> gpurun_out/g16_bench.err
tail -3 gpurun_out/g16_pytest.log; python -c "
import json; d=json.loads(open('gpurun_out/g16_bench.json').read().splitlines()[-1]); print(d['value'], d['e2e'])"
