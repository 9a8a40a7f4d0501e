cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_skeletons.py -x -q -k "policy" > gpurun_out/g28_pytest.log 2>&1; tail -3 gpurun_out/g28_pytest.log
timeout 1200 python bench.py --no-cpu --no-extras --e2e-steps 0 > gpurun_out/g28_bench.json 2>/dev/null; cut -c1-200 gpurun_out/g28_bench.json
timeout 1200 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/g28_launches.csv \
    python bench.py --steps 2 --warmup 3 --e2e-steps 0 --no-cpu > gpurun_out/g28_launches_bench.json 2> gpurun_out/g28_launches.err
ls ~/.cache/skel_b200/*.policy | head; cat ~/.cache/skel_b200/*.policy | head -40
