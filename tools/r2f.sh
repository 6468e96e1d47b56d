mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_r2f.log 2>&1 || { tail gpurun_out/build_r2f.log; exit 1; }
timeout 1800 python -m pytest tests/test_gpu_cheby.py tests/test_gpu_campaign.py tests/test_gpu_sr.py tests/test_gpu_tiled.py tests/test_gpu_dist1.py -q --tb=short --durations=5 > gpurun_out/tests_r2f.log 2>&1; tail -15 gpurun_out/tests_r2f.log
for rep in 1 2; do timeout 300 python tools/spmv_time.py --reps 200 2>&1 | tail -1; done > gpurun_out/var_r2f.log; cat gpurun_out/var_r2f.log
