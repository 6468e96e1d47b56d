"""Design-time check of the two folded-index SECDED layouts frozen in DESIGN.md §3
(not product/oracle code): distance-4 (all singles located, all doubles detected)
and invertibility of the reserved-bit submatrix."""
import itertools

def e96_col(b):
    w, j = divmod(b, 32)
    if w == 0: return j | (0 << 5)
    if w == 1: return j | ((1 | (2 if j == 31 else 0)) << 5)
    # col word
    if j < 24: return j | (2 << 5)
    pos = {24: 8, 25: 17}.get(j, j)
    code = {24: 3, 25: 3, 26: 3, 27: 3, 28: 3, 29: 2, 30: 2, 31: 1}[j]
    return pos | (code << 5)

def v64_col(b):
    w, j = divmod(b, 32)
    if w == 1: return j | (1 << 5)
    if j >= 8: return j
    pos = {1: 9, 2: 18}.get(j, j)
    code = [0, 2, 2, 2, 0, 0, 0, 3][j]
    return pos | (code << 5)

for name, W, colf, reserved in [("E96", 96, e96_col, range(88, 96)), ("V64", 64, v64_col, range(0, 8))]:
    cols = [colf(b) for b in range(W)]
    assert len(set(cols)) == W, name
    assert cols.count(0) == 1
    # doubles: q = 0 and s = c_a ^ c_b != 0 always since distinct
    for a, b in itertools.combinations(range(W), 2):
        assert cols[a] ^ cols[b] != 0
    # reserved rank with q row
    basis = []
    for b in reserved:
        v = cols[b] | (1 << 7)
        for x in basis: v = min(v, v ^ x)
        assert v, (name, b)
        basis.append(v)
    print(name, "ok: zero-column bit", cols.index(0), "reserved rank", len(basis))
