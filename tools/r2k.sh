#!/bin/bash
# A/B of SpMV variants on one box (tools/spmv_time.py, 2 rounds each) + tiled parity tests
mkdir -p gpurun_out
T=${T:-r2k}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$T.log 2>&1 || { tail gpurun_out/build_$T.log; exit 1; }
if [ -n "$TESTS" ]; then timeout 1800 python -m pytest $TESTS -q --tb=short --maxfail=5 > gpurun_out/tests_$T.log 2>&1; tail -15 gpurun_out/tests_$T.log; fi
for rep in 1 2; do
for v in $VARIANTS; do
  ABFT_SO=variants/libabft_$v.so timeout 300 python tools/spmv_time.py --reps 100 --schemes ${SCHEMES:-2,0} 2>&1 | tail -1
done
done > gpurun_out/ab_$T.jsonl
python - <<'PY'
import json, os
T = os.environ.get("T", "r2k")
for l in open(f"gpurun_out/ab_{T}.jsonl"):
    try: d = json.loads(l)
    except Exception: print(l[:200]); continue
    print(d["so"].split("/")[-1], {k: (round(v["spmv_ms"], 4), round(v.get("spmv_partials_ms", 0), 4), round(v["calc_ur_ms"], 4), round(v["calc_p_ms"], 4), round(v["cg_step_ms_200it"] / 200, 4)) for k, v in d.items() if k != "so"})
PY
