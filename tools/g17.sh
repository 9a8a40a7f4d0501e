cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for d in "-DMANDEL_PERIODIC=1 -DMANDEL_PRE=8" "-DMANDEL_PERIODIC=1 -DMANDEL_PRE=16" "-DMANDEL_PERIODIC=1 -DMANDEL_PRE=8 -DMANDEL_B=4" "-DMANDEL_PERIODIC=1 -DMANDEL_PRE=8 -DMANDEL_B=16" "-DMANDEL_PERIODIC=1 -DMANDEL_PRE=4 -DMANDEL_B=4"; do SKEL_NVRTC_DEFINES="$d" timeout 300 python tools/mandel_probe.py >> gpurun_out/g17_mandel.jsonl 2>&1; done
cat gpurun_out/g17_mandel.jsonl
