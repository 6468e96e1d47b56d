mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_r2h.log 2>&1 || { tail gpurun_out/build_r2h.log; exit 1; }
timeout 2700 python -m pytest tests -m gpu -q --tb=short --maxfail=20 --durations=15 > gpurun_out/tests_r2h.log 2>&1; tail -25 gpurun_out/tests_r2h.log
timeout 300 python __graft_entry__.py --smoke > gpurun_out/smoke_r2h.log 2>&1; tail -2 gpurun_out/smoke_r2h.log
bash tools/r2g.sh r2h
