#!/bin/bash
# Map at small sizes: grid policy / cache-hint variants vs the hand-written float4 kernel.
cd "${GRAFT_REPO_ROOT:-/root/repo}"; mkdir -p gpurun_out
export PROBE_OPS=map
S="18 20 21 22 23 24"
echo base; timeout 300 python tools/small_n_probe.py $S
echo per_thread1; SKEL_EW_PER_THREAD=1 timeout 300 python tools/small_n_probe.py $S
echo waves1; SKEL_EW_WAVES=1 timeout 300 python tools/small_n_probe.py $S
echo st_default; SKEL_NVRTC_DEFINES='-DSKEL_ST_HINT=' timeout 300 python tools/small_n_probe.py $S
echo ld_nc; SKEL_NVRTC_DEFINES='-DSKEL_LD_HINT=.nc -DSKEL_ST_HINT=' timeout 300 python tools/small_n_probe.py $S
