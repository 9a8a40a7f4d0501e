cd "${GRAFT_REPO_ROOT:-/root/repo}"
timeout 900 python -m pytest tests -m gpu -x -q -k "skeleton or mandel or distrib or lmosem" > gpurun_out/g27_pytest.log 2>&1; tail -2 gpurun_out/g27_pytest.log
mkdir -p gpurun_out
for i in 1 2; do SKEL_LOG=1 timeout 1200 python bench.py --no-cpu > gpurun_out/g27_bench_$i.json 2> gpurun_out/g27_bench_$i.err; done
for i in 1 2; do python -c "
import json; d=json.loads(open('gpurun_out/g27_bench_$i.json').read().splitlines()[-1]); m=d['mandelbrot']
print(d['value'], {k:round(v['ms'],4) for k,v in d['per_skeleton'].items()}, d['e2e']['value'])
print(d['overhead']['small']['2^20'], d['overhead']['small']['2^22'])
print(m['variants_ms']); print(m['configs0_1024x768']['variants_ms']); print(m['cap4096']['ms']); print(d['lmosem']['subset_s'])"; done
grep "grid policy, size class 2[23]" gpurun_out/g27_bench_*.err | sort | uniq -c | head -60
