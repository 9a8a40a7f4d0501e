cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_skeletons.py tests/test_gpu_mandelbrot.py tests/test_gpu_lmosem.py tests/test_gpu_graphs.py -m gpu -q -x > gpurun_out/g20_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g20_pytest.log
timeout 1200 python bench.py --no-cpu > gpurun_out/g20_bench.json 2> gpurun_out/g20_bench.err
tail -3 gpurun_out/g20_pytest.log
python -c "
import json; d=json.loads(open('gpurun_out/g20_bench.json').read().splitlines()[-1]); m=d['mandelbrot']
print(d['value'], {k:round(v['ms'],4) for k,v in d['per_skeleton'].items()}, d['e2e']['value'])
print(d['overhead']['small'])
print([(r['log2n'], {k:r[k]['frac'] for k in ('map','zip','reduce','scan')}) for r in d['sweep'] if r['dtype']=='float32'])
print(m['variants_ms']); print(m['configs0_1024x768']['variants_ms']); print(m['cap4096']['ms'])
print(d['lmosem']['subset_s'], d['lmosem']['given_order'], d['lmosem']['roofline']['map_ms'], d['lmosem']['roofline']['device_order']['map_ms'])"
