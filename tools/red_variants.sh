#!/bin/bash
# Reduce/Scan variants across sizes: tools/small_n_probe.py per variant.
# VARIANTS holds lines `run <label> "<nvrtc defines>" "<env assignments>"`.
cd "${GRAFT_REPO_ROOT:-/root/repo}"; mkdir -p gpurun_out
out=gpurun_out/red_variants.jsonl; : > $out
run() {  # label, defines, env
  echo "{\"variant\": \"$1\", \"defines\": \"$2\", \"env\": \"$3\"}" >> $out
  env $3 SKEL_NVRTC_DEFINES="$2" timeout 300 python tools/small_n_probe.py ${SIZES:-20 22 24 26 28 30} >> $out 2>&1
}
if [ -n "$VARIANTS" ]; then eval "$VARIANTS"; else run base "" ""; fi
cat $out
