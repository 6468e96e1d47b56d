#!/bin/bash
# full GPU tests, SpMV variant A/B, CRC interval sweep (default vs L1 slicing tables), bench
mkdir -p gpurun_out
T=${T:-r2m}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw,power.limit --format=csv > gpurun_out/gpu_$T.txt
T=$T VARIANTS="$VARIANTS" TESTS="$TESTS" bash tools/r2k.sh
if [ -n "$CRC" ]; then
  for so in default $(echo $CRC | sed "s/^-$//"); do
    if [ $so = default ]; then unset ABFT_SO; else export ABFT_SO=variants/libabft_$so.so; fi
    timeout 900 python tools/sweep.py --grid 8192 --iters 200 --no-schemes --intervals 1,128 --only CRC32C,SECDED64 \
      --out gpurun_out/sweep_crc_${so}_$T.json > gpurun_out/sweep_crc_${so}_$T.log 2>&1
    echo "== $so"; grep -o '"scheme": "[A-Z0-9]*".*"check_interval": [0-9]*, "iter_ms": [0-9.]*, "overhead_pct": [-0-9.]*' gpurun_out/sweep_crc_${so}_$T.log | sed 's/"elem.*"check_interval"/ N/'
  done
  unset ABFT_SO
fi
if [ -n "$BENCH" ]; then
  timeout 900 python bench.py > gpurun_out/bench_$T.json 2> gpurun_out/bench_$T.err; tail -2 gpurun_out/bench_$T.err; cat gpurun_out/bench_$T.json
fi
