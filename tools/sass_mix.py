import csv, sys, collections
rows = list(csv.reader(open(sys.argv[1])))
hdr = rows[1]
iA, iS, iE, iW = hdr.index("Address"), hdr.index("Source"), hdr.index("Instructions Executed"), hdr.index("Warp Stall Sampling (All Samples)")
tot = 0; ops = collections.Counter(); samp = collections.Counter(); tots=0
seq = []
for r in rows[2:]:
    if len(r) <= iE: continue
    try: e = int(r[iE]); s = int(r[iW])
    except: continue
    src = r[iS].strip()
    op = src.split()[0] if not src.startswith("@") else src.split()[1]
    op = op.split(".")[0]
    ops[op] += e; samp[op] += s; tot += e; tots += s
    seq.append((r[iA], src, e, s))
print("total warp inst", tot, "samples", tots)
for op, e in ops.most_common(40):
    print(f"{op:12s} {e/1e6:8.2f}M {100*e/tot:5.1f}%  stall-samples {100*samp[op]/tots:5.1f}%")
