#!/bin/bash
# Round profiling pass (one GPU): launch list of the bench command, ncu --set full
# of the four skeleton kernels at 2^30 and of the two workload Maps.
cd "${GRAFT_REPO_ROOT:-/root/repo}"; mkdir -p gpurun_out
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv \
    python bench.py --steps 2 --warmup 3 --e2e-steps 0 --no-cpu > gpurun_out/launches_bench.json 2> gpurun_out/launches.err
ncu --set full --clock-control none --import-source on -k 'regex:skel_(ew|reduce|scan)_kernel' -s 12 -c 4 \
    -o gpurun_out/prof_skel python bench.py --steps 1 --warmup 3 --e2e-steps 0 --no-cpu --no-extras > gpurun_out/prof_skel.log 2>&1
ncu --set full --clock-control none --import-source on -k regex:skel_ew_kernel -s 2 -c 1 \
    -o gpurun_out/prof_lm python tools/lmosem_scaling_proxy.py > gpurun_out/prof_lm.log 2>&1
ncu --set full --clock-control none --import-source on -k regex:skel_ew_kernel -s 2 -c 1 \
    -o gpurun_out/prof_mandel python tools/workload_once.py mandel > gpurun_out/prof_mandel.log 2>&1
ls -la gpurun_out
