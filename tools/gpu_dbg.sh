# r32: DRAM bytes of the default (3-D TMA window) k_spmv_tile from a single-pass
# metric capture (no kernel replay), and application-replay attempt of the sections
mkdir -p gpurun_out
N="--steps 1 --warmup 0 --no-e2e --no-cpu-baseline --no-fused-extra --max-iters 4"
timeout 400 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k regex:'k_spmv_tile|k_calc' -s 6 -c 6 --csv --log-file gpurun_out/dram_r32.csv python bench.py $N > gpurun_out/ncu_dram_r32.log 2>&1; tail -2 gpurun_out/ncu_dram_r32.log; cat gpurun_out/dram_r32.csv | cut -c1-220 | tail -20
timeout 900 ncu --replay-mode application --section SpeedOfLight --section MemoryWorkloadAnalysis --section Occupancy --clock-control none -k regex:'k_spmv_tile' -s 6 -c 1 -o gpurun_out/prof_r32app -f python bench.py $N > gpurun_out/ncu_app_r32.log 2>&1; tail -3 gpurun_out/ncu_app_r32.log
