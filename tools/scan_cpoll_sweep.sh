#!/bin/bash
# coalesced status polling (SKEL_SCAN_CPOLL) vs the strided probes: parity, then timing
cd "${GRAFT_REPO_ROOT:-/root/repo}"; mkdir -p gpurun_out
SKEL_NVRTC_DEFINES="-DSKEL_SCAN_CPOLL=1" timeout 900 python -m pytest tests -m gpu -x -q -k "scan or Scan or fullsize" > gpurun_out/cpoll_tests.log 2>&1; echo "tests $?" >> gpurun_out/cpoll_tests.log
bash tools/scan_variants.sh "" "-DSKEL_SCAN_CPOLL=1" "-DSKEL_SCAN_CPOLL=1 -DSKEL_SCAN_REPL=16" "-DSKEL_SCAN_REPL=16" "-DSKEL_SCAN_CPOLL=1 -DSKEL_SCAN_LAG=3" "-DSKEL_SCAN_CPOLL=1 -DSKEL_SCAN_BACKOFF_MAX=256" "-DSKEL_SCAN_CPOLL=1 -DSKEL_SCAN_REPL=4" "" "-DSKEL_SCAN_CPOLL=1" 2>&1 | tee gpurun_out/cpoll_sweep.txt
