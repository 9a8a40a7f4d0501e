#!/bin/bash
# session-4 follow-up: scan knobs with coalesced probes, and the small/persistent crossover
cd "${GRAFT_REPO_ROOT:-/root/repo}"; mkdir -p gpurun_out
bash tools/scan_variants.sh "" "-DSKEL_SCAN_CH=2" "-DSKEL_SCAN_LAG=1" "-DSKEL_SCAN_REPL=2" "-DSKEL_SCAN_REPL=2 -DSKEL_SCAN_BACKOFF_MIN=16 -DSKEL_SCAN_BACKOFF_MAX=128" "-DSKEL_SCAN_NPRE=8" "" "-DSKEL_SCAN_REPL=2" > gpurun_out/s4_sweep.txt 2>&1
timeout 300 python tools/small_n_probe.py 20 21 22 23 24 > gpurun_out/small_default.txt 2>&1
SKEL_SCAN_SMALL_MAX=0 timeout 300 python tools/small_n_probe.py 20 21 22 23 24 > gpurun_out/small_persistent.txt 2>&1
