"""Fault-injection campaign (BASELINE.json config 5; S§8(c) O10, S§8(d)).

    python tools/campaign.py [--grid 4096] [--rates 1e-9,1e-8,1e-7,1e-6,1e-5] [--seeds 20]
                             [--kind single|double|both] [--arms secded,sed] [--out gpurun_out/campaign.json]

Per trial, on the GPU through the C ABI: encode the G-TEA matrix and the five
CG vectors b, x, r, p, w (arm "secded": E-SECDED + R-SECDED64 + V-SECDED64, the
config-2 schemes; arm "sed": E-SECDED + R-SED + V-SED, the SDC contrast arm),
draw K ~ Binomial(words, rate) storage words uniformly over val (64-bit), col,
rowptr (32-bit) and the vectors (64-bit) from splitmix64(seed), flip one bit
(single) or two distinct bits of the same word (double) at each, run
`abft_check_all` (scrub) of the matrix and b, x, r, p, then ONE protected SpMV
w = A p (which overwrites w).

Parity: for grids the oracle can afford (<= 512^2 by default) the same trial is
run by the ORACLE on its own encoding of the raw inputs (or_check_csr +
or_vec_check, then or_spmv): both count sets, the SpMV output words and all
scrubbed storage must be bit-identical.  At 4096^2 the check_all counts are
compared with the oracle's own check of every touched codeword (every other
codeword is clean and contributes nothing; the rowptr range-violation tally is
the range rule start <= end <= nnz on the masked stored entries, validated
against the full oracle at 512^2), and in single-flip trials (everything
scrubbed) the SpMV must report nothing and reproduce the oracle's clean 4096^2
SpMV output word for word.

Ground truth classifies every flipped storage word after the trial:
  masked     — in w, overwritten by the SpMV before any read;
  corrected  — stored word back to its clean value (single-bit correction);
  due        — still corrupted and its codeword fails the code's check;
  sdc        — still corrupted but its codeword passes the check (silent data
               corruption: undetected and the value used differs).
"""
from __future__ import annotations

import argparse
import json
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import gen  # noqa: E402

ARMS = {"secded": ("SECDED64", "SECDED64", "SECDED64"), "sed": ("SECDED64", "SED", "SED")}


def binomial(seed: int, words: int, rate: float) -> int:
    """K ~ Binomial(words, rate), the generator seeded from splitmix64(seed)."""
    s = int(gen.splitmix64(np.array([0], dtype=np.uint64), seed)[0])
    return int(np.random.Generator(np.random.PCG64(s)).binomial(words, rate))


def draw_words(seed: int, k: int, words: int) -> np.ndarray:
    """k distinct word indices in [0, words) from splitmix64."""
    out, i = [], 0
    seen = set()
    while len(out) < k:
        cand = gen.splitmix64(np.arange(i, i + 2 * k + 8, dtype=np.uint64), seed ^ 0x5EED) % np.uint64(words)
        for c in cand.tolist():
            if c not in seen:
                seen.add(c)
                out.append(c)
                if len(out) == k:
                    break
        i += 2 * k + 8
    return np.array(out, dtype=np.int64)


def draw_flips(kind, rate, seed, segs):
    """[(segment, word, [bits])] for one trial."""
    words = sum(s[1] for s in segs)
    k = binomial(seed * 1000003 + int(rate * 1e12), words, rate)
    widx = draw_words(seed * 7919 + int(-np.log10(rate) * 13) + (kind == "double"), k, words)
    bits = gen.splitmix64(np.arange(2 * k, dtype=np.uint64), seed + 99).reshape(-1, 2) if k else \
        np.zeros((0, 2), dtype=np.uint64)
    out = []
    for t, w in enumerate(widx.tolist()):
        b0 = 0
        for name, cnt_w, wb in segs:
            if b0 <= w < b0 + cnt_w:
                b_a = int(bits[t, 0] % np.uint64(wb))
                bl = [b_a]
                if kind == "double":
                    b_b = int(bits[t, 1] % np.uint64(wb - 1))
                    bl.append(b_b + 1 if b_b >= b_a else b_b)
                out.append((name, w - b0, bl))
                break
            b0 += cnt_w
    return out


def run(grid, rates, seeds, kinds, out_path, arms=("secded", "sed"), full_oracle=None, verbose=True):
    import torch
    import oracle as orc
    from paper_conf_cluster_pawelczakmpm17_b200 import abft
    n = grid
    N = n * n
    nnz = 5 * N
    full = (grid <= 512) if full_oracle is None else full_oracle
    dev = torch.device("cuda", 0)
    ctx = abft.Context(0)
    val_d, col_d, rp_d = gen.tealeaf_csr(n, device=dev)
    col_d, rp_d = col_d.to(torch.int32), rp_d.to(torch.int32)
    vec_vals = [gen.tealeaf_rhs(n, device=dev)] + [torch.from_numpy(gen.uniform_pm1(N, 100 + j)).to(dev)
                                                  for j in range(4)]
    val_h, col_h, rp_h = val_d.cpu().numpy(), col_d.cpu().numpy().view(np.uint32), rp_d.cpu().numpy().view(np.uint32)
    vec_h = [v.cpu().numpy() for v in vec_vals]
    results = []
    for arm in arms:
        ES, RS, VS = (getattr(abft, s) for s in ARMS[arm])
        A = abft.Matrix(val_d.clone(), col_d.clone(), rp_d, N, N, ES, RS, stencil_n=n if n % 256 == 0 else 0)
        rp_len = A.rowptr.numel()
        npad = orc.vec_padded_len(N, VS)
        segs = [("val", nnz, 64), ("col", nnz, 32), ("rowptr", rp_len, 32)] + \
               [(f"v{j}", N, 64) for j in range(5)]
        words = sum(s[1] for s in segs)
        # clean encodings, by the oracle from the raw inputs (ground truth)
        Ac = orc.Matrix(val_h.copy(), col_h.copy(), rp_h.copy(), N, N, ES, RS)
        assert Ac.encode() == 0
        vc = [orc.vec_encode(v, VS) for v in vec_h]
        clean_out = None   # the oracle's SpMV of the clean problem (large grids, computed once)
        for kind in kinds:
            for rate in rates:
                for seed in range(1, seeds + 1):
                    t0 = time.time()
                    A.val.copy_(val_d)
                    A.col.copy_(col_d)
                    A.rowptr.zero_()
                    A.rowptr[:N + 1].copy_(rp_d)
                    assert A.encode(ctx) == 0
                    vecs = [abft.Vector.from_values(ctx, v, VS) for v in vec_vals]
                    enc_ok = (np.array_equal(A.col.cpu().numpy().view(np.uint32), Ac.col) and
                              np.array_equal(A.rowptr.cpu().numpy().view(np.uint32), Ac.rowptr) and
                              all(np.array_equal(v.words().cpu().numpy().view(np.uint64), c) for v, c in zip(vecs, vc)))
                    flips = draw_flips(kind, rate, seed, segs)
                    for (name, wi, bl) in flips:
                        for b in bl:
                            if name == "val":
                                abft.inject_bitflip(ctx, A.val, 64 * wi + b)
                            elif name == "col":
                                abft.inject_bitflip(ctx, A.col, 32 * wi + b)
                            elif name == "rowptr":
                                abft.inject_bitflip(ctx, A.rowptr, 32 * wi + b)
                            else:
                                abft.inject_bitflip(ctx, vecs[int(name[1:])].data, 64 * wi + b)
                    c_sp, c_ck = abft.Counters(), abft.Counters()
                    abft.check_all(ctx, A, vecs[:4], c_ck, scrub=True)
                    abft.spmv(ctx, A, vecs[3], vecs[4], c_sp)
                    torch.cuda.synchronize()
                    g_sp, g_ck = c_sp.read(), c_ck.read()
                    g_val = A.val.view(torch.int64).cpu().numpy().view(np.uint64)
                    g_col = A.col.cpu().numpy().view(np.uint32)
                    g_rp = A.rowptr.cpu().numpy().view(np.uint32)
                    g_vec = [v.words().cpu().numpy().view(np.uint64) for v in vecs]
                    rec = {"arm": arm, "kind": kind, "rate": rate, "seed": seed, "flips": len(flips),
                           "encode_match": enc_ok}
                    # ---- parity vs the oracle
                    if full:
                        Ao = _clone(orc, Ac)
                        vo = [c.copy() for c in vc]
                        for (name, wi, bl) in flips:
                            for b in bl:
                                if name == "val":
                                    Ao.val[wi] ^= np.uint64(1 << b)
                                elif name == "col":
                                    Ao.col[wi] ^= np.uint32(1 << b)
                                elif name == "rowptr":
                                    Ao.rowptr[wi] ^= np.uint32(1 << b)
                                else:
                                    vo[int(name[1:])][wi] ^= np.uint64(1 << b)
                        o_sp, o_ck = orc.new_counts(), orc.new_counts()
                        Ao.check(o_ck)
                        for v in vo[:4]:
                            orc.vec_check(v, N, VS, o_ck)
                        orc.spmv(Ao, vo[3], N, VS, vo[4], N, o_sp)
                        rec["oracle_match"] = bool(
                            np.array_equal(g_sp, o_sp) and np.array_equal(g_ck, o_ck) and
                            np.array_equal(g_val, Ao.val) and np.array_equal(g_col, Ao.col) and
                            np.array_equal(g_rp, Ao.rowptr) and
                            all(np.array_equal(g[:npad], o[:npad]) for g, o in zip(g_vec, vo)))
                    else:
                        ok = bool(np.array_equal(g_ck, _touched_counts(orc, flips, Ac, vc, ES, RS, VS, N, nnz)))
                        if kind == "single" and arm == "secded":
                            if clean_out is None:
                                clean_out = _clean_spmv(orc, Ac, vc, VS, N)
                            ok = ok and not g_sp.any() and np.array_equal(g_vec[4][:N], clean_out[:N])
                        rec["oracle_match"] = ok
                    # ---- ground-truth classification of every flipped word
                    cls = {"masked": 0, "corrected": 0, "due": 0, "sdc": 0}
                    for (name, wi, bl) in flips:
                        cls[_classify(orc, name, wi, Ac, vc, g_val, g_col, g_rp, g_vec, ES, RS, VS, N)] += 1
                    rec.update(cls)
                    rec["detected"] = int((g_sp + g_ck)[:, :, 0].sum())
                    rec["corrected_count"] = int((g_sp + g_ck)[:, :, 1].sum())
                    rec["uncorrectable"] = int((g_sp + g_ck)[:, :, 2].sum())
                    rec["seconds"] = round(time.time() - t0, 2)
                    results.append(rec)
                    if verbose:
                        print(json.dumps(rec), flush=True)
    summary = {"grid": grid, "trials": len(results), "full_oracle": full,
               "all_match_oracle": all(r["oracle_match"] for r in results),
               "all_encodings_match": all(r["encode_match"] for r in results)}
    for arm in arms:
        for kind in kinds:
            rs = [r for r in results if r["arm"] == arm and r["kind"] == kind]
            summary[f"{arm}_{kind}"] = {k: sum(r[k] for r in rs) for k in ("flips", "masked", "corrected", "due", "sdc")}
    if out_path:
        os.makedirs(os.path.dirname(out_path) or ".", exist_ok=True)
        json.dump({"summary": summary, "trials": results}, open(out_path, "w"), indent=1)
    if verbose:
        print(json.dumps(summary))
    return summary, results


def _codeword_state(orc, name, wi, words_val, words_col, words_rp, words_vec, ES, RS, VS, N):
    """The oracle's check of the (final) codeword holding storage word wi of
    `name`: CLEAN / CORRECTED (correctable) / DUE."""
    if name in ("val", "col"):
        M = orc.Matrix(words_val[wi:wi + 1].view(np.float64).copy(), words_col[wi:wi + 1].copy(), np.array([0, 1], dtype=np.uint32),
                       1, 1 << 24, ES, orc.NONE)
        c = orc.new_counts()
        M.check(c, scrub=False)
        if c[orc.ELEM, ES, orc.UNC]:
            return orc.DUE
        return orc.CORRECTED if c[orc.ELEM, ES, orc.COR] else orc.CLEAN
    if name == "rowptr":
        G = {orc.SED: 1, orc.SECDED64: 2}[RS]
        g0 = wi // G * G
        ents = words_rp[g0:g0 + G].copy().astype(np.uint32)
        if RS == orc.SED:
            return orc.CLEAN if bin(int(ents[0])).count("1") % 2 == 0 else orc.DUE
        o, _ = orc.secded_check(orc.I_R_SECDED64, ents)
        return o
    w = words_vec[0 if name == "v" else int(name[1:])][wi:wi + 1].copy()
    c = orc.new_counts()
    orc.vec_check(w, 1, VS, c, scrub=False)
    if c[orc.VEC, VS, orc.UNC]:
        return orc.DUE
    return orc.CORRECTED if c[orc.VEC, VS, orc.COR] else orc.CLEAN


def _classify(orc, name, wi, Ac, vc, g_val, g_col, g_rp, g_vec, ES, RS, VS, N):
    if name == "v4":
        return "masked"          # w: written by the SpMV before any read
    if name == "val":
        clean = g_val[wi] == Ac.val[wi] and g_col[wi] == Ac.col[wi]
    elif name == "col":
        clean = g_col[wi] == Ac.col[wi] and g_val[wi] == Ac.val[wi]
    elif name == "rowptr":
        clean = g_rp[wi] == Ac.rowptr[wi]
    else:
        clean = g_vec[int(name[1:])][wi] == vc[int(name[1:])][wi]
    if clean:
        return "corrected"
    st = _codeword_state(orc, name, wi, g_val, g_col, g_rp, g_vec, ES, RS, VS, N)
    return "sdc" if st == orc.CLEAN else "due"


def _clone(orc, Ac):
    """An oracle matrix holding exactly Ac's stored words (padding included)."""
    M = orc.Matrix(Ac.val.view(np.float64).copy(), Ac.col.copy(), Ac.rowptr.copy(), Ac.nrows, Ac.ncols, Ac.es, Ac.rs)
    M.rowptr[:] = Ac.rowptr
    M.nnz = Ac.nnz    # (the constructor read nnz from rowptr[nrows], which now carries ECC bits)
    return M


def _clean_spmv(orc, Ac, vc, VS, N):
    """The oracle's SpMV w = A p of the clean encoded problem."""
    M = _clone(orc, Ac)
    out = np.zeros(len(vc[3]), dtype=np.uint64)
    orc.spmv(M, vc[3].copy(), N, VS, out, N, None)
    return out


def _touched_counts(orc, flips, Ac, vc, ES, RS, VS, N, nnz):
    """Expected check_all counters of one trial (large grids) from the oracle's
    check of every touched codeword of the matrix and b, x, r, p (w is not
    checked: the SpMV overwrites it)."""
    G = {orc.SED: 1, orc.SECDED64: 2}[RS]
    groups = {}
    for (name, wi, bl) in flips:
        if name == "v4":
            continue
        key = ("el", wi) if name in ("val", "col") else ("rp", wi // G) if name == "rowptr" else (name, wi)
        groups.setdefault(key, []).append((name, wi, bl))
    exp = orc.new_counts()
    dues_rp = {}
    for key, fl in groups.items():
        if key[0] == "el":
            v, c = Ac.val[key[1]:key[1] + 1].copy(), Ac.col[key[1]:key[1] + 1].copy()
            for (name, wi, bl) in fl:
                for b in bl:
                    if name == "val":
                        v[0] ^= np.uint64(1 << b)
                    else:
                        c[0] ^= np.uint32(1 << b)
            st = _codeword_state(orc, "val", 0, v, c, None, None, ES, RS, VS, N)
            t, s = orc.ELEM, ES
            # a DUE element keeps its stored bits: check_all range-checks the masked stored column
            if st == orc.DUE and (int(c[0]) & (0x7FFFFFFF if ES == orc.SED else 0x00FFFFFF)) >= N:
                exp[orc.ELEM, ES, orc.RANGE] += 1
        elif key[0] == "rp":
            g0 = key[1] * G
            ents = Ac.rowptr[g0:g0 + G].copy()
            for (name, wi, bl) in fl:
                for b in bl:
                    ents[wi - g0] ^= np.uint32(1 << b)
            st = _codeword_state(orc, "rowptr", 0, None, None, ents, None, ES, RS, VS, N)
            t, s = orc.ROWPTR, RS
            if st != orc.CORRECTED:   # DUE, or an undetected (even-weight SED) change: stored bits are used
                for q in range(G):
                    dues_rp[g0 + q] = int(ents[q]) & (0x7FFFFFFF if RS == orc.SED else 0x0FFFFFFF)
        else:
            j = int(key[0][1:])
            w = vc[j][key[1]:key[1] + 1].copy()
            for (name, wi, bl) in fl:
                for b in bl:
                    w[0] ^= np.uint64(1 << b)
            st = _codeword_state(orc, "v", 0, None, None, None, [w], ES, RS, VS, N)
            t, s = orc.VEC, VS
        if st != orc.CLEAN:
            exp[t, s, orc.DET] += 1
            exp[t, s, orc.COR if st == orc.CORRECTED else orc.UNC] += 1
    # check_all's row pass: the range rule on the masked stored entries of row pointers left corrupted
    rows = set()
    for i in dues_rp:
        rows.update(r_ for r_ in (i - 1, i) if 0 <= r_ < N)
    for r_ in rows:
        s_ = dues_rp.get(r_, int(Ac.rowptr[r_]) & (0x7FFFFFFF if RS == orc.SED else 0x0FFFFFFF))
        t_ = dues_rp.get(r_ + 1, int(Ac.rowptr[r_ + 1]) & (0x7FFFFFFF if RS == orc.SED else 0x0FFFFFFF))
        if not (s_ <= t_ <= nnz):
            exp[orc.ROWPTR, RS, orc.RANGE] += 1
    return exp


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--grid", type=int, default=4096)
    ap.add_argument("--rates", default="1e-9,1e-8,1e-7,1e-6,1e-5")
    ap.add_argument("--seeds", type=int, default=20)
    ap.add_argument("--kind", default="both", choices=["single", "double", "both"])
    ap.add_argument("--arms", default="secded,sed")
    ap.add_argument("--out", default=os.path.join(ROOT, "gpurun_out", "campaign.json"))
    a = ap.parse_args()
    kinds = ["single", "double"] if a.kind == "both" else [a.kind]
    run(a.grid, [float(x) for x in a.rates.split(",")], a.seeds, kinds, a.out, arms=a.arms.split(","))


if __name__ == "__main__":
    main()
