# round-2 measurement session: bench, ncu (launch list + full capture of the
# dominant kernel, its twin and the BLAS-1 kernels, exported to CSV on the box
# so gpurun_out stays small), config-3 sweep, config-4 at N=1, config-5 campaign
mkdir -p gpurun_out
T=${1:-r2g}
WHAT=${2:-"bench ncu sweep strong campaign"}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
export_rep() {   # $1 = report base name: raw + source CSV, then drop the binary report
  ncu -i gpurun_out/$1.ncu-rep --page raw --csv > gpurun_out/$1_raw.csv 2>/dev/null
  ncu -i gpurun_out/$1.ncu-rep --page source --csv --print-source cuda,sass > gpurun_out/$1_src.csv 2>/dev/null
  rm -f gpurun_out/$1.ncu-rep
}
for w in $WHAT; do case $w in
bench)
  timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json ;;
ncu)
  timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_$T.csv \
    python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --no-fused-extra --no-sr-extra --max-iters 30 > gpurun_out/ncu_launch_bench_$T.json 2>&1
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv_tile' -s 3 -c 1 \
    -o gpurun_out/prof_tma_prot_$T -f python tools/spmv_time.py --reps 2 --schemes 2 > gpurun_out/ncu_tma_prot_$T.log 2>&1
  export_rep prof_tma_prot_$T
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv_tile' -s 3 -c 1 \
    -o gpurun_out/prof_tma_twin_$T -f python tools/spmv_time.py --reps 2 --schemes 0 > gpurun_out/ncu_tma_twin_$T.log 2>&1
  export_rep prof_tma_twin_$T
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_calc_ur|k_calc_p' -s 4 -c 2 \
    -o gpurun_out/prof_blas_$T -f python tools/spmv_time.py --reps 2 --schemes 2 > gpurun_out/ncu_blas_$T.log 2>&1
  export_rep prof_blas_$T
  ls -la gpurun_out/*_$T* | head -30 ;;
sweep)
  timeout 1500 python tools/sweep.py --out gpurun_out/sweep_$T.json --intervals 1,8,32,128 > gpurun_out/sweep_$T.log 2>&1; tail -3 gpurun_out/sweep_$T.log ;;
strong)
  timeout 1200 python bench.py --mode strong --steps 2 --warmup 3 --no-cpu-baseline --no-fused-extra --no-sr-extra > gpurun_out/bench_strong_$T.json 2> gpurun_out/bench_strong_$T.err; cat gpurun_out/bench_strong_$T.json ;;
campaign)
  timeout 2400 python tools/campaign.py --grid 4096 --seeds 4 --out gpurun_out/campaign_4096_$T.json > gpurun_out/campaign_$T.log 2>&1; tail -2 gpurun_out/campaign_$T.log ;;
esac; done
du -sh gpurun_out
