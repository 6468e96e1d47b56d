# same-box A/B of calc_p variants (tools/build_variant.sh): base, full unroll, full unroll + minb 5
mkdir -p gpurun_out
for rep in 1 2 3; do for v in base p1u p1u5; do echo "== $v"; ABFT_SO=variants/libabft_$v.so timeout 300 python tools/spmv_time.py --reps 200 2>&1 | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print(d['scheme2']['calc_p_ms'], d['scheme0']['calc_p_ms'])"; done; done
