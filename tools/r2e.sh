set -x
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_r2e.log 2>&1 || { tail gpurun_out/build_r2e.log; exit 1; }
for rep in 1 2; do
  timeout 300 python tools/spmv_time.py --reps 200 2>&1 | tail -1
  ABFT_NO_PERSIST=1 timeout 300 python tools/spmv_time.py --reps 200 2>&1 | tail -1
done > gpurun_out/var_r2e.log
cat gpurun_out/var_r2e.log
timeout 2400 python -m pytest tests/test_gpu_tiled.py tests/test_gpu_geometry.py tests/test_gpu_fused.py tests/test_gpu_loopback.py tests/test_gpu_faults.py tests/test_gpu_sr.py tests/test_gpu_interval.py tests/test_gpu_parity.py tests/test_gpu_crc_fix.py -q --tb=short --durations=5 -x > gpurun_out/tests_r2e.log 2>&1; tail -12 gpurun_out/tests_r2e.log
