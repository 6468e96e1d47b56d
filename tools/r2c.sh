set -x
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_r2c.log 2>&1 || { tail gpurun_out/build_r2c.log; exit 1; }
for rep in 1 2; do for v in base earlywin noticket; do ABFT_SO=variants/libabft_$v.so timeout 300 python tools/spmv_time.py --reps 200 2>&1 | tail -1; done; done > gpurun_out/var_r2c.log
cat gpurun_out/var_r2c.log
timeout 1500 python -m pytest tests/test_gpu_campaign.py "tests/test_gpu_geometry.py::test_8192_five_chunk_spmv_sampled" tests/test_gpu_faults.py tests/test_gpu_tiled.py tests/test_gpu_fused.py -q --tb=short --durations=10 -x > gpurun_out/tests_r2c.log 2>&1; tail -15 gpurun_out/tests_r2c.log
