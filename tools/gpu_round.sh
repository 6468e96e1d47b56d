#!/bin/bash
# One GPU session: tests, smoke, bench, ncu launch list + full capture of the
# hot kernels.  Usage (under gpurun): bash tools/gpu_round.sh [tag] [what...]
TAG=${1:-r01}; shift
WHAT=${@:-"tests smoke bench ncu"}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/gpu_$TAG.txt
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$TAG.log 2>&1 || { cat gpurun_out/build_$TAG.log; exit 1; }
for w in $WHAT; do
  case $w in
  tests)
    timeout 2400 python -m pytest tests -m gpu -q --tb=short --maxfail=30 --durations=25 > gpurun_out/tests_$TAG.log 2>&1
    tail -30 gpurun_out/tests_$TAG.log ;;
  smoke)
    timeout 300 python __graft_entry__.py --smoke > gpurun_out/smoke_$TAG.log 2>&1; tail -5 gpurun_out/smoke_$TAG.log ;;
  bench)
    timeout 900 python bench.py > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err; tail -3 gpurun_out/bench_$TAG.err; cat gpurun_out/bench_$TAG.json ;;
  benchref)
    timeout 900 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/benchref_$TAG.json 2>&1; cat gpurun_out/benchref_$TAG.json ;;
  ncu)
    timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_$TAG.csv \
      python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --max-iters 30 > gpurun_out/ncu_launch_bench_$TAG.json 2>&1
    timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv|k_calc_ur|k_calc_p' -s 6 -c 6 \
      -o gpurun_out/prof_$TAG -f python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --max-iters 4 > gpurun_out/ncu_full_$TAG.log 2>&1
    tail -3 gpurun_out/ncu_full_$TAG.log ;;
  ncuspmv)
    timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv' -s 2 -c 4 \
      -o gpurun_out/prof_$TAG -f python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --max-iters 3 > gpurun_out/ncu_full_$TAG.log 2>&1
    tail -3 gpurun_out/ncu_full_$TAG.log ;;
  sanitize)
    for tool in memcheck racecheck synccheck initcheck; do
      timeout 1500 compute-sanitizer --tool $tool --print-limit 20 --error-exitcode 9 python tools/sanitize_run.py \
        > gpurun_out/sanitize_${tool}_$TAG.log 2>&1
      echo "$tool rc=$?"; tail -4 gpurun_out/sanitize_${tool}_$TAG.log
    done ;;
  ncutma)
    # kernel-replay capture of the DEFAULT (3-D TMA window) protected SpMV and its unprotected twin
    timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv_tile' -s 3 -c 1 \
      -o gpurun_out/prof_tma_prot_$TAG -f python tools/spmv_time.py --reps 2 --schemes 2 > gpurun_out/ncu_tma_prot_$TAG.log 2>&1
    tail -3 gpurun_out/ncu_tma_prot_$TAG.log
    timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv_tile' -s 3 -c 1 \
      -o gpurun_out/prof_tma_twin_$TAG -f python tools/spmv_time.py --reps 2 --schemes 0 > gpurun_out/ncu_tma_twin_$TAG.log 2>&1
    tail -3 gpurun_out/ncu_tma_twin_$TAG.log ;;
  sweep)
    timeout 1500 python tools/sweep.py --out gpurun_out/sweep_$TAG.json > gpurun_out/sweep_$TAG.log 2>&1; tail -4 gpurun_out/sweep_$TAG.log ;;
  big)
    timeout 1200 python bench.py --grid 16384 --steps 2 --warmup 3 --max-iters 3000 --no-cpu-baseline > gpurun_out/bench16k_$TAG.json 2> gpurun_out/bench16k_$TAG.err
    tail -3 gpurun_out/bench16k_$TAG.err; cat gpurun_out/bench16k_$TAG.json ;;
  esac
done
