#!/bin/bash
# A/B (variants on one box), ncu source-level capture of the default protected
# SpMV, default bench
mkdir -p gpurun_out
T=${T:-r2l}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
T=$T VARIANTS="$VARIANTS" bash tools/r2k.sh
if [ -n "$NCU" ]; then
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv_tile' -s 3 -c 1 \
    -o gpurun_out/prof_prot_$T -f python tools/spmv_time.py --reps 2 --schemes 2 > gpurun_out/ncu_prot_$T.log 2>&1
  ncu -i gpurun_out/prof_prot_$T.ncu-rep --page raw --csv > gpurun_out/prof_prot_${T}_raw.csv 2>/dev/null
  ncu -i gpurun_out/prof_prot_$T.ncu-rep --page source --csv --print-source cuda,sass > gpurun_out/prof_prot_${T}_src.csv 2>/dev/null
  rm -f gpurun_out/prof_prot_$T.ncu-rep
  python tools/ncu_lines.py gpurun_out/prof_prot_${T}_src.csv > gpurun_out/ncu_lines_$T.txt 2>&1; head -40 gpurun_out/ncu_lines_$T.txt
fi
if [ -n "$BENCH" ]; then
  timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; tail -2 gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json
fi
