"""Design-time search for the E-SECDED (96-bit CSR element) folded-index layout.

Not part of the product or the oracle: it only explores candidate H-matrix
layouts and prints the ones that satisfy the SECDED + invertibility constraints
(DESIGN.md §3.2 explains the structure).  Container words: A = val[0:32],
B = val[32:64], C = col (reserved C[24:32]).
Rows: q (all ones), s0..s4 = 5-bit "index" of the bit's fold position,
s5, s6 = code rows.
"""
import itertools

def rank_gf2(vecs):
    rows = list(vecs); r = 0
    basis = []
    for v in rows:
        for b in basis:
            v = min(v, v ^ b)
        if v:
            basis.append(v); r += 1
    return r

def cols_for(t1, t2, res_codes, bswap, cdata_code=0b10):
    """Return list of 96 (index, code) pairs (code = s5 | s6<<1)."""
    cols = []
    for j in range(32):                     # A
        cols.append((j, 0b00))
    for j in range(32):                     # B
        cols.append((j, bswap.get(j, 0b01)))
    for j in range(24):                     # C data
        cols.append((j, cdata_code))
    for t in range(8):                      # C reserved
        if t == t1: idx = 8 + t
        elif t == t2: idx = 16 + t
        else: idx = 24 + t
        cols.append((idx, res_codes[t]))
    return cols

def full(col):
    idx, code = col
    return 1 | (idx << 1) | (code << 6)     # q | s0..s4 | s5 s6

def ok(cols):
    f = [((c[0]) | (c[1] << 5)) for c in cols]   # 7-bit syndrome column
    if len(set(f)) != 96: return False
    if f.count(0) != 1: return False
    return rank_gf2([full(c) for c in cols[88:]]) == 8

if __name__ != "__main__":
    raise SystemExit
found = 0
for t1 in range(8):
    for t2 in range(8):
        if t1 == t2: continue
        for swap_idx in [None] + list(range(24, 32)):
            for swap_code in (0b11, 0b10):
                bswap = {} if swap_idx is None else {swap_idx: swap_code}
                for codes in itertools.product(range(4), repeat=8):
                    cols = cols_for(t1, t2, codes, bswap)
                    if ok(cols):
                        found += 1
                        if found <= 40:
                            print("t1", t1, "t2", t2, "bswap", bswap, "codes", codes)
                if swap_idx is None: break
print("found", found)
