#!/bin/bash
# session j baseline: HEAD kernels timed alone (twice) and the default bench
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_r2j.log 2>&1 || { tail gpurun_out/build_r2j.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_r2j.txt
for rep in 1 2; do timeout 300 python tools/spmv_time.py --reps 100 2>&1 | tail -1; done > gpurun_out/spmv_time_r2j.jsonl
cat gpurun_out/spmv_time_r2j.jsonl
timeout 900 python bench.py > gpurun_out/bench_r2j.json 2> gpurun_out/bench_r2j.err; cat gpurun_out/bench_r2j.json
