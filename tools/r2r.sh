#!/bin/bash
# bulk-staged calc_p: parity tests, A/B, bench, sanitizers, ncu of the BLAS-1 kernels
mkdir -p gpurun_out
T=${T:-r2r}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
timeout 2400 python -m pytest $TESTS -q --tb=short --maxfail=5 > gpurun_out/tests_$T.log 2>&1; tail -3 gpurun_out/tests_$T.log
T=$T VARIANTS="$VARIANTS" bash tools/r2k.sh
timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; tail -2 gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json
if [ -n "$SAN" ]; then
  for tool in memcheck racecheck synccheck initcheck; do
    timeout 1500 compute-sanitizer --tool $tool --print-limit 20 --error-exitcode 9 python tools/sanitize_run.py \
      > gpurun_out/sanitize_${tool}_$T.log 2>&1
    echo "$tool rc=$?"; tail -3 gpurun_out/sanitize_${tool}_$T.log
  done
fi
