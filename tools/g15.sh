cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for i in 1 2 3; do timeout 600 python bench.py --no-extras --no-cpu --e2e-steps 0 --steps 10 >> gpurun_out/g15_bench.jsonl 2>/dev/null; done
python - <<'PY' > gpurun_out/g15_summary.txt
import json
for ln in open("gpurun_out/g15_bench.jsonl"):
    d = json.loads(ln)
    print(round(d["value"], 1), {k: round(v["ms"], 4) for k, v in d["per_skeleton"].items()})
PY
for t in memcheck racecheck synccheck initcheck; do echo "## $t" >> gpurun_out/g15_san.txt; timeout 1500 compute-sanitizer --tool $t --print-limit 20 python tools/sanitize_run.py >> gpurun_out/g15_san.txt 2>&1; echo "rc=$?" >> gpurun_out/g15_san.txt; done
cat gpurun_out/g15_summary.txt; grep -E "^## |SUMMARY|FAILED|all ok|rc=" gpurun_out/g15_san.txt
