#!/bin/bash
# usage (on the GPU box): bash tools/scan_lab_run.sh "<opts1>" "<opts2>" ...  -- times each, traces the first
cd "${GRAFT_REPO_ROOT:-/root/repo}"; mkdir -p gpurun_out
D=paper_conf_ipps_steuwerkg11_b200/csrc/skeletons
first=1
for o in "$@"; do
  if [ $first = 1 ]; then
    timeout 120 ./tools/scan_lab $D 30 5 gpurun_out/scan_trace.bin $o; first=0
    python tools/scan_trace.py gpurun_out/scan_trace.bin
  fi
  timeout 120 ./tools/scan_lab $D 30 20 - $o
done
