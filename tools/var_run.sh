#!/bin/bash
# usage: bash var_run.sh "v1 v2 ..." [tests]
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/vbuild.log 2>&1 || { tail gpurun_out/vbuild.log; exit 1; }
if [ -n "$2" ]; then timeout 900 python -m pytest $2 -q -x 2>&1 | tail -3; fi
for rep in 1 2; do
for v in $1; do
  ABFT_SO=variants/libabft_$v.so timeout 300 python tools/spmv_time.py --reps 100 2>&1 | tail -1
done
done
