#!/bin/bash
# tests after the default changes, kernel timing, range-mode CRC vs SECDED SpMV (timing + ncu), bench
mkdir -p gpurun_out
T=${T:-r2n}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
timeout 1800 python -m pytest $TESTS -q --tb=short --maxfail=5 > gpurun_out/tests_$T.log 2>&1; tail -3 gpurun_out/tests_$T.log
for m in 0 2; do
  timeout 300 python tools/spmv_time.py --reps 100 --schemes 2/2/0,4/4/0,1/1/0,0/0/0 --mode $m --spmv-only 2>&1 | tail -1
done > gpurun_out/range_$T.jsonl; cat gpurun_out/range_$T.jsonl
for sc in 4/4/0 2/2/0; do
  tag=$(echo $sc | tr / _)
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv_tile' -s 3 -c 1 \
    -o gpurun_out/prof_range_${tag}_$T -f python tools/spmv_time.py --reps 2 --schemes $sc --mode 2 --spmv-only > gpurun_out/ncu_range_${tag}_$T.log 2>&1
  ncu -i gpurun_out/prof_range_${tag}_$T.ncu-rep --page raw --csv > gpurun_out/prof_range_${tag}_${T}_raw.csv 2>/dev/null
  ncu -i gpurun_out/prof_range_${tag}_$T.ncu-rep --page source --csv --print-source cuda,sass > gpurun_out/prof_range_${tag}_${T}_src.csv 2>/dev/null
  rm -f gpurun_out/prof_range_${tag}_$T.ncu-rep
  python tools/ncu_lines.py gpurun_out/prof_range_${tag}_${T}_src.csv 25 > gpurun_out/ncu_lines_range_${tag}_$T.txt 2>&1
done
for rep in 1 2; do timeout 300 python tools/spmv_time.py --reps 100 2>&1 | tail -1; done > gpurun_out/spmv_time_$T.jsonl
timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; tail -2 gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json
