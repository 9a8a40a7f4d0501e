cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_lmosem.py tests/test_gpu_graphs.py tests/test_gpu_fused.py tests/test_gpu_scan_progress.py -m gpu -q -x > gpurun_out/g3_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/g3_pytest.log
timeout 900 python tools/lmosem_scaling_proxy.py > gpurun_out/g3_proxy.jsonl 2> gpurun_out/g3_proxy.err
M=l1tex__t_sector_pipe_lsu_mem_global_op_ld_hit_rate.pct,l1tex__t_sector_hit_rate.pct,l1tex__t_requests_pipe_lsu_mem_global_op_ld.sum,l1tex__t_requests_pipe_lsu_mem_global_op_red.sum,gpu__time_duration.sum,sm__warps_active.avg.pct_of_peak_sustained_active,smsp__thread_inst_executed_per_inst_executed.ratio
timeout 600 ncu --kernel-name skel_ew_kernel --launch-skip 2 --launch-count 1 --metrics $M --csv python tools/workload_once.py lmosem > gpurun_out/g3_ncu_given.csv 2> gpurun_out/g3_ncu.err
timeout 600 ncu --kernel-name skel_ew_kernel --launch-skip 6 --launch-count 1 --metrics $M --csv python tools/workload_once.py lmosem_device > gpurun_out/g3_ncu_device.csv 2>> gpurun_out/g3_ncu.err
tail -3 gpurun_out/g3_pytest.log; cat gpurun_out/g3_proxy.jsonl; tail -12 gpurun_out/g3_ncu_given.csv; tail -12 gpurun_out/g3_ncu_device.csv
