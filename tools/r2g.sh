# round-2 measurement session: bench, ncu (launch list + full capture of the
# dominant kernel and its twin), config-3 sweep, config-5 campaign, config-4 at N=1
mkdir -p gpurun_out
T=${1:-r2g}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_$T.csv \
  python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --no-fused-extra --max-iters 30 > gpurun_out/ncu_launch_bench_$T.json 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv_tile' -s 3 -c 1 \
  -o gpurun_out/prof_tma_prot_$T -f python tools/spmv_time.py --reps 2 --schemes 2 > gpurun_out/ncu_tma_prot_$T.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv_tile' -s 3 -c 1 \
  -o gpurun_out/prof_tma_twin_$T -f python tools/spmv_time.py --reps 2 --schemes 0 > gpurun_out/ncu_tma_twin_$T.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_calc_ur|k_calc_p' -s 4 -c 2 \
  -o gpurun_out/prof_blas_$T -f python tools/spmv_time.py --reps 2 --schemes 2 > gpurun_out/ncu_blas_$T.log 2>&1
timeout 1500 python tools/sweep.py --out gpurun_out/sweep_$T.json --intervals 1,8,32,128 > gpurun_out/sweep_$T.log 2>&1; tail -3 gpurun_out/sweep_$T.log
timeout 1200 python bench.py --mode strong --steps 2 --warmup 3 --no-cpu-baseline --no-fused-extra > gpurun_out/bench_strong_$T.json 2> gpurun_out/bench_strong_$T.err; cat gpurun_out/bench_strong_$T.json
timeout 2400 python tools/campaign.py --grid 4096 --seeds 4 --out gpurun_out/campaign_4096_$T.json > gpurun_out/campaign_$T.log 2>&1; tail -2 gpurun_out/campaign_$T.log
