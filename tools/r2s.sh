#!/bin/bash
# G > 1 / CRC pass-loop unroll A/B, bench, launch list + ncu of the bulk calc_p
mkdir -p gpurun_out
T=${T:-r2s}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
if [ -n "$TESTS" ]; then timeout 2400 python -m pytest $TESTS -q --tb=short --maxfail=5 > gpurun_out/tests_$T.log 2>&1; tail -3 gpurun_out/tests_$T.log; fi
for rep in 1 2; do for v in $VARIANTS; do
  ABFT_SO=variants/libabft_$v.so timeout 300 python tools/spmv_time.py --reps 50 --schemes 3,4,2/2/3,2/2/4,2 --spmv-only 2>&1 | tail -1
done; done > gpurun_out/ab_g1_$T.jsonl; cat gpurun_out/ab_g1_$T.jsonl
timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; tail -2 gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_$T.csv \
  python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --no-fused-extra --no-sr-extra --max-iters 30 > gpurun_out/ncu_launch_bench_$T.json 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_calc_p' -s 2 -c 2 \
  -o gpurun_out/prof_calcp_$T -f python tools/spmv_time.py --reps 2 --schemes 2 > gpurun_out/ncu_calcp_$T.log 2>&1
ncu -i gpurun_out/prof_calcp_$T.ncu-rep --page raw --csv > gpurun_out/prof_calcp_${T}_raw.csv 2>/dev/null
rm -f gpurun_out/prof_calcp_$T.ncu-rep
