"""Aggregate an ncu source page (--print-source cuda,sass --csv) by CUDA
source line: warp-stall samples and executed warp instructions per line.

    ncu -i rep.ncu-rep --page source --csv --print-source cuda,sass > mix.csv
    python tools/ncu_lines.py mix.csv [top]
"""
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
top = int(sys.argv[2]) if len(sys.argv) > 2 else 40
agg = {}
cur_file = None
hdr = None
tot_s = tot_i = 0
for r in rows:
    if not r:
        continue
    if r[0] == "File Path":
        cur_file = r[1].split("/")[-1]
        continue
    if r[0] == "Line No":
        hdr = r
        continue
    if hdr is None or len(r) < 8:
        continue
    try:
        line = int(r[0])
        samp = int(r[4] or 0)
        inst = int(r[7] or 0)
    except ValueError:
        continue
    key = (cur_file, line)
    s, i, src = agg.get(key, (0, 0, r[1].strip()[:70]))
    agg[key] = (s + samp, i + inst, src)
    tot_s += samp
    tot_i += inst
print(f"total samples {tot_s}, warp instructions {tot_i}")
for (f, l), (s, i, src) in sorted(agg.items(), key=lambda kv: -kv[1][0])[:top]:
    print(f"{f:18s}:{l:5d}  samples {100 * s / max(tot_s, 1):5.1f}%  inst {100 * i / max(tot_i, 1):5.1f}%  {src}")
