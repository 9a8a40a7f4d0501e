cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1200 python bench.py --no-cpu > gpurun_out/g19_bench.json 2> gpurun_out/g19_bench.err
python -c "
import json; d=json.loads(open('gpurun_out/g19_bench.json').read().splitlines()[-1]); m=d['mandelbrot']
print(d['value'], d['e2e']['value'], d['e2e']['ms_per_step']); print(m['variants_ms']); print(m['configs0_1024x768']); print(m['cap4096']['ms'])"
