cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_mandelbrot.py -m gpu -q -x -k pairs > gpurun_out/g23_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g23_pytest.log
timeout 1200 python bench.py --no-cpu > gpurun_out/g23_bench.json 2> gpurun_out/g23_bench.err
tail -2 gpurun_out/g23_pytest.log
python -c "
import json; d=json.loads(open('gpurun_out/g23_bench.json').read().splitlines()[-1]); m=d['mandelbrot']
print(d['value'], {k:round(v['ms'],4) for k,v in d['per_skeleton'].items()}, d['e2e']['value'])
print(d['overhead']['small']['2^20'], d['overhead']['small']['2^22'])
print(m['variants_ms']); print(m['configs0_1024x768']['variants_ms']); print(m['cap4096']['ms'])"
