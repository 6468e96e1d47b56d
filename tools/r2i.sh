mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_r2i.log 2>&1 || { tail gpurun_out/build_r2i.log; exit 1; }
timeout 1800 python -m pytest tests/test_gpu_ppcg.py tests/test_gpu_crc_fix.py tests/test_gpu_cheby.py tests/test_gpu_sr.py "tests/test_gpu_loopback.py::test_loopback_single_reduction_cg" tests/test_gpu_faults.py -q --tb=short --durations=5 > gpurun_out/tests_r2i.log 2>&1; tail -15 gpurun_out/tests_r2i.log
bash tools/r2g.sh r2i "ncu sweep campaign"
