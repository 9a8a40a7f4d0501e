cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for i in 1 2; do timeout 600 python bench.py --no-cpu --no-extras --e2e-steps 0 --steps 10 >> gpurun_out/g21_bench.jsonl 2>/dev/null; done
python - <<'PY'
import json
for ln in open("gpurun_out/g21_bench.jsonl"):
    d = json.loads(ln); print(round(d["value"], 1), {k: round(v["ms"], 4) for k, v in d["per_skeleton"].items()})
PY
timeout 300 python tools/mandel_probe.py
