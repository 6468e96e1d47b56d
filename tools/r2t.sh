#!/bin/bash
# final: full GPU suite + smoke on the final defaults, bench, ncu launch list
mkdir -p gpurun_out
T=${T:-r2t}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
timeout 2400 python -m pytest tests -m gpu -q --tb=short --maxfail=10 > gpurun_out/tests_$T.log 2>&1; tail -3 gpurun_out/tests_$T.log
timeout 300 python __graft_entry__.py --smoke > gpurun_out/smoke_$T.log 2>&1; tail -2 gpurun_out/smoke_$T.log
for rep in 1 2; do timeout 300 python tools/spmv_time.py --reps 100 2>&1 | tail -1; done > gpurun_out/spmv_time_$T.jsonl
timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; tail -2 gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_$T.csv \
  python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --no-fused-extra --no-sr-extra --max-iters 30 > gpurun_out/ncu_launch_bench_$T.json 2>&1
