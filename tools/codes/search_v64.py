"""Design-time search for the V-SECDED64 folded-index layout (not product/oracle code).

Container: A = bits 0..31 (reserved A[0:8]), B = bits 32..63.
Rows: q, s0..s4 (fold index), s5, s6 (code rows).  Reserved bits t1, t2 are
moved to fold positions 8+t1 / 16+t2 (one PRMT replicating byte 0).
Scores layouts by the number of ones in the inverse of the 8x8 reserved
matrix (= XOR work of the encoder) and prints the best.
"""
import itertools

def gf2_inv(cols):
    """cols: list of 8 ints (8-bit columns). Return inverse as list of 8 columns or None."""
    n = 8
    # matrix M[row][col]
    M = [[(cols[c] >> r) & 1 for c in range(n)] for r in range(n)]
    I = [[int(r == c) for c in range(n)] for r in range(n)]
    for c in range(n):
        p = next((r for r in range(c, n) if M[r][c]), None)
        if p is None: return None
        M[c], M[p] = M[p], M[c]; I[c], I[p] = I[p], I[c]
        for r in range(n):
            if r != c and M[r][c]:
                M[r] = [a ^ b for a, b in zip(M[r], M[c])]
                I[r] = [a ^ b for a, b in zip(I[r], I[c])]
    return I

def layout(t1, t2, codes, bswap):
    cols = []
    for j in range(32):
        if j < 8:
            idx = 8 + j if j == t1 else (16 + j if j == t2 else j)
            cols.append((idx, codes[j]))
        else:
            cols.append((j, 0))
    for j in range(32):
        cols.append((j, bswap.get(j, 1)))
    return cols

def check(cols):
    f = [c[0] | (c[1] << 5) for c in cols]
    if len(set(f)) != 64 or f.count(0) != 1: return None
    full = [1 | (c[0] << 1) | (c[1] << 6) for c in cols[:8]]
    return gf2_inv(full)

if __name__ == "__main__":
    best = []
    for t1 in range(8):
        for t2 in range(8):
            if t1 == t2: continue
            for codes in itertools.product(range(4), repeat=8):
                inv = check(layout(t1, t2, codes, {}))
                if inv is None: continue
                ones = sum(map(sum, inv))
                best.append((ones, t1, t2, codes))
    best.sort()
    print(len(best))
    for b in best[:25]: print(b)
