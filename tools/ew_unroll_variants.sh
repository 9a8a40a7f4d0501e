#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
export PROBE_OPS=map,zip
S="20 22 24 26 28 30"
echo "unroll1"; timeout 300 python tools/small_n_probe.py $S
echo "compiler"; SKEL_NVRTC_DEFINES='-DSKEL_MAIN_UNROLL=' timeout 300 python tools/small_n_probe.py $S
echo "unroll1_U8"; SKEL_NVRTC_DEFINES='-DSKEL_UNROLL=8' timeout 300 python tools/small_n_probe.py $S
