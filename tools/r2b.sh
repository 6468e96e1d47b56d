set -x
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_r2b.log 2>&1 || { tail gpurun_out/build_r2b.log; exit 1; }
timeout 1500 python -m pytest tests/test_gpu_faults.py tests/test_gpu_campaign.py "tests/test_gpu_geometry.py::test_8192_five_chunk_spmv_sampled" -q --tb=short --durations=10 > gpurun_out/tests_r2b.log 2>&1; tail -25 gpurun_out/tests_r2b.log
ABFT_SO=variants/libabft_rpf2m4.so timeout 900 python -m pytest tests/test_gpu_tiled.py "tests/test_gpu_geometry.py::test_tiled_spmv_1024_cross_tile" tests/test_gpu_interval.py -q --tb=short -x > gpurun_out/tests_r2b_var.log 2>&1; tail -5 gpurun_out/tests_r2b_var.log
for rep in 1 2; do for v in base rpf2m4 rpf; do ABFT_SO=variants/libabft_$v.so timeout 300 python tools/spmv_time.py --reps 200 2>&1 | tail -1; done; done > gpurun_out/var_r2b.log
cat gpurun_out/var_r2b.log
