# r31: tests, bench, variant timing of the TMA window, launch list and a full
# ncu capture on the LDG-window path (ncu kernel replay of the 3-D TMA window
# kernel fails with LaunchFailed)
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_r31.log 2>&1 || { tail gpurun_out/build_r31.log; exit 1; }
timeout 1200 python -m pytest tests -m gpu -q --tb=short --maxfail=30 > gpurun_out/tests_r31.log 2>&1; tail -3 gpurun_out/tests_r31.log
timeout 300 python __graft_entry__.py --smoke 2>&1 | tail -1
timeout 900 python bench.py > gpurun_out/bench_r31.json 2> gpurun_out/bench_r31.err; cat gpurun_out/bench_r31.json
for rep in 1 2; do echo "== tma"; timeout 300 python tools/spmv_time.py --reps 100 2>&1 | tail -1; echo "== ldg"; ABFT_NO_VMAPS=1 timeout 300 python tools/spmv_time.py --reps 100 2>&1 | tail -1; done
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_r31.csv \
  python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --no-fused-extra --max-iters 30 > gpurun_out/ncu_launch_bench_r31.json 2>&1
ABFT_NO_VMAPS=1 timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_spmv|k_calc_ur|k_calc_p' -s 6 -c 6 \
  -o gpurun_out/prof_r31 -f python bench.py --steps 1 --warmup 0 --no-e2e --no-cpu-baseline --no-fused-extra --max-iters 4 > gpurun_out/ncu_full_r31.log 2>&1
tail -3 gpurun_out/ncu_full_r31.log
