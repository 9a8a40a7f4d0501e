#!/bin/bash
# One gpurun call: all GPU tests, smoke, bench (default args), reference arm, the
# bench's launch list and ncu --set full of the four skeleton kernels at 2^30 and of
# three Mandelbrot forms (paper loop, periodic, lockstep pairs + periodic).
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
T=${TAG:-full}
timeout 3000 python -m pytest tests -m gpu -q -rs > gpurun_out/${T}_pytest.log 2>&1; echo "pytest rc=$?" >> gpurun_out/${T}_pytest.log
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${T}_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/${T}_smoke.log
timeout 1200 python bench.py > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err; echo "bench rc=$?" >> gpurun_out/${T}_bench.err
timeout 600 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/${T}_bench_ref.json 2> gpurun_out/${T}_bench_ref.err
timeout 1200 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/${T}_launches.csv \
    python bench.py --steps 2 --warmup 3 --e2e-steps 0 --no-cpu > gpurun_out/${T}_launches_bench.json 2> gpurun_out/${T}_launches.err
timeout 900 ncu --set full --clock-control none --import-source on --nvtx --nvtx-include timed/ -k regex:skel_ew_kernel -c 2 \
    -o gpurun_out/${T}_prof_ew -f python bench.py --steps 1 --warmup 3 --e2e-steps 0 --no-cpu --no-extras > gpurun_out/${T}_prof_ew.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --nvtx --nvtx-include timed/ -k 'regex:skel_(reduce|scan)_kernel' -c 2 \
    -o gpurun_out/${T}_prof_rs -f python bench.py --steps 1 --warmup 3 --e2e-steps 0 --no-cpu --no-extras > gpurun_out/${T}_prof_rs.log 2>&1
timeout 900 python tools/lmosem_scaling_proxy.py > gpurun_out/${T}_proxy.jsonl 2> gpurun_out/${T}_proxy.err
for v in paper periodic pairs_periodic; do
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:skel_ew -s 3 -c 1 \
      -o gpurun_out/${T}_mandel_$v -f python tools/mandel_one.py $v 128 > gpurun_out/${T}_mandel_$v.log 2>&1
done
tail -3 gpurun_out/${T}_pytest.log; tail -2 gpurun_out/${T}_smoke.log; cut -c1-400 gpurun_out/${T}_bench.json; tail -2 gpurun_out/${T}_bench.err
