#!/bin/bash
# session-3 final measurement: full GPU suite, variant A/B, bench, ncu (launch
# list + full captures exported to CSV), config-3 sweep, config 4 at N = 1
mkdir -p gpurun_out
T=${T:-r2q}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
timeout 2400 python -m pytest tests -m gpu -q --tb=short --maxfail=10 > gpurun_out/tests_$T.log 2>&1; tail -3 gpurun_out/tests_$T.log
timeout 300 python __graft_entry__.py --smoke > gpurun_out/smoke_$T.log 2>&1; tail -2 gpurun_out/smoke_$T.log
T=$T VARIANTS="$VARIANTS" bash tools/r2k.sh
timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; tail -2 gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json
bash tools/r2g.sh $T "ncu strong sweep"
