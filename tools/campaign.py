"""Fault-injection campaign (BASELINE.json config 5; S§8(d)).

    python tools/campaign.py [--grid 4096] [--rates 1e-9,1e-8,1e-7,1e-6,1e-5] [--seeds 20]
                             [--kind single|double|both] [--out gpurun_out/campaign.json]

Per trial: encode the G-TEA matrix (E-SECDED + R-SECDED64) and the five CG
vectors b, x, r, p, w (V-SECDED64) on the GPU, draw K ~ Binomial(words, rate)
storage words uniformly over val (64-bit), col, rowptr (32-bit) and the vectors
(64-bit) from splitmix64(seed), flip one bit (single) or two distinct bits of
the same word (double) at each, run `abft_check_all` (scrub) and one protected
SpMV, and compare the detected / corrected / uncorrectable counts bit-exactly
with the CPU oracle.  The oracle is evaluated only on the codewords the flips
touched (every other codeword is clean and contributes nothing), encoding each
one from the generator's raw values itself — no oracle input comes from the
GPU.  Ground truth also classifies every flip as corrected / DUE / SDC.
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


def binomial(seed: int, words: int, rate: float) -> int:
    """K ~ Binomial(words, rate) from splitmix64 (inverse-CDF via Poisson
    approximation is exact enough for rate <= 1e-5; use numpy's generator
    seeded from splitmix64 for the draw itself)."""
    s = int(gen.splitmix64(np.array([0], dtype=np.uint64), seed)[0])
    return int(np.random.Generator(np.random.PCG64(s)).binomial(words, rate))


def draw_words(seed: int, k: int, words: int) -> np.ndarray:
    """k distinct word indices in [0, words)."""
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


def run(grid, rates, seeds, kinds, out_path, check_spmv=True):
    import torch
    import oracle as orc
    from paper_conf_cluster_pawelczakmpm17_b200 import abft
    S = abft.SECDED64
    n = grid
    N = n * n
    dev = torch.device("cuda", 0)
    ctx = abft.Context(0)
    val, col, rowptr = gen.tealeaf_csr(n, device=dev)
    col = col.to(torch.int32)
    rowptr = rowptr.to(torch.int32)
    nnz = 5 * N
    val0 = val.clone()   # pristine values: DUE'd (unscrubbed) flips must not leak into the next trial
    A = abft.Matrix(val.clone(), col.clone(), rowptr, N, N, S, S, stencil_n=n if n % 256 == 0 else 0)
    rp_len = A.rowptr.numel()
    vec_vals = [gen.tealeaf_rhs(n, device=dev)] + [torch.from_numpy(gen.uniform_pm1(N, 100 + j)).to(dev)
                                                  for j in range(4)]
    # storage-word map: val (nnz x 64), col (nnz x 32), rowptr (rp_len x 32), 5 vectors (N x 64)
    segs = [("val", nnz, 64), ("col", nnz, 32), ("rowptr", rp_len, 32)] + [(f"v{j}", N, 64) for j in range(5)]
    words = sum(s[1] for s in segs)
    # host copies of the raw inputs for the oracle's own encoding of touched codewords
    val_h = val.cpu().numpy()
    col_h = col.cpu().numpy().view(np.uint32)
    rp_h = rowptr.cpu().numpy().view(np.uint32)
    vec_h = [v.cpu().numpy() for v in vec_vals]
    results = []
    for kind in kinds:
        for rate in rates:
            for seed in range(1, seeds + 1):
                t0 = time.time()
                A.val.copy_(val0)
                A.col.copy_(col)
                A.rowptr.zero_()
                A.rowptr[:N + 1].copy_(rowptr)
                assert A.encode(ctx) == 0
                vecs = [abft.Vector.from_values(ctx, v, S) for v in vec_vals]
                k = binomial(seed * 1000003 + int(rate * 1e12), words, rate)
                widx = draw_words(seed * 7919 + int(-np.log10(rate) * 13) + (kind == "double"), k, words)
                bits = gen.splitmix64(np.arange(2 * k, dtype=np.uint64), seed + 99).reshape(-1, 2) if k else \
                    np.zeros((0, 2), dtype=np.uint64)
                # --- apply on the GPU and collect the oracle codewords
                touched = {}   # (target, codeword id) -> list of (segment, word, bit)
                base = 0
                bounds = []
                for name, cnt_w, wb in segs:
                    bounds.append((name, base, cnt_w, wb))
                    base += cnt_w
                for t, w in enumerate(widx.tolist()):
                    for name, b0, cnt_w, wb in bounds:
                        if b0 <= w < b0 + cnt_w:
                            wi = w - b0
                            nb = 1 if kind == "single" else 2
                            b_a = int(bits[t, 0] % np.uint64(wb))
                            b_list = [b_a]
                            if nb == 2:
                                b_b = int(bits[t, 1] % np.uint64(wb - 1))
                                b_list.append(b_b + 1 if b_b >= b_a else b_b)
                            for bb in b_list:
                                if name == "val":
                                    abft.inject_bitflip(ctx, A.val, 64 * wi + bb)
                                    key = ("el", wi)
                                elif name == "col":
                                    abft.inject_bitflip(ctx, A.col, 32 * wi + bb)
                                    key = ("el", wi)
                                elif name == "rowptr":
                                    abft.inject_bitflip(ctx, A.rowptr, 32 * wi + bb)
                                    key = ("rp", wi // 2)
                                else:
                                    j = int(name[1:])
                                    abft.inject_bitflip(ctx, vecs[j].data, 64 * wi + bb)
                                    key = (name, wi)
                                touched.setdefault(key, []).append((name, wi, bb))
                            break
                cnt = abft.Counters()
                abft.check_all(ctx, A, vecs, cnt, scrub=True)
                gpu_counts = cnt.read()
                # --- oracle on the touched codewords only
                oc = orc.new_counts()
                bad_rp = {}
                for key, fl in touched.items():
                    if key[0] == "el":
                        e = key[1]
                        row = e // 5
                        M = orc.Matrix(val_h[e:e + 1], col_h[e:e + 1], np.array([0, 1], dtype=np.uint32), 1, N,
                                       orc.SECDED64, orc.NONE)
                        M.encode()
                        for (name, wi, bb) in fl:
                            if name == "val":
                                M.val[0] ^= np.uint64(1 << bb)
                            else:
                                M.col[0] ^= np.uint32(1 << bb)
                        c1 = orc.new_counts()
                        M.check(c1)
                        oc[orc.ELEM] += c1[orc.ELEM]
                        del row
                    elif key[0] == "rp":
                        g = key[1]
                        ents = np.array([rp_h[2 * g] if 2 * g <= N else nnz,
                                         rp_h[2 * g + 1] if 2 * g + 1 <= N else nnz], dtype=np.uint32)
                        wv = orc.secded_encode(orc.I_R_SECDED64, ents)
                        for (name, wi, bb) in fl:
                            wv[wi - 2 * g] ^= np.uint32(1 << bb)
                        stored = wv.copy()
                        o, _ = orc.secded_check(orc.I_R_SECDED64, wv)
                        if o != orc.CLEAN:
                            oc[orc.ROWPTR, orc.SECDED64, orc.DET] += 1
                            oc[orc.ROWPTR, orc.SECDED64, orc.COR if o == orc.CORRECTED else orc.UNC] += 1
                        if o == orc.DUE:   # masked stored entries stay in place: row range checks see them
                            bad_rp[2 * g] = int(stored[0]) & 0x0FFFFFFF
                            bad_rp[2 * g + 1] = int(stored[1]) & 0x0FFFFFFF
                    else:
                        j = int(key[0][1:])
                        wv = orc.vec_encode(vec_h[j][key[1]:key[1] + 1], orc.SECDED64)
                        for (name, wi, bb) in fl:
                            wv[0] ^= np.uint64(1 << bb)
                        orc.vec_check(wv, 1, orc.SECDED64, oc)
                # check_all's row pass: start <= end <= nnz on the (possibly DUE) entries
                rows = set()
                for i in bad_rp:
                    rows.update(r_ for r_ in (i - 1, i) if 0 <= r_ < N)
                for r_ in rows:
                    s_ = bad_rp.get(r_, int(rp_h[r_]))
                    t_ = bad_rp.get(r_ + 1, int(rp_h[r_ + 1]) if r_ + 1 <= N else nnz)
                    if not (s_ <= t_ <= nnz):
                        oc[orc.ROWPTR, orc.SECDED64, orc.RANGE] += 1
                ok = bool(np.array_equal(gpu_counts, oc))
                det = int(gpu_counts[:, :, 0].sum())
                cor = int(gpu_counts[:, :, 1].sum())
                unc = int(gpu_counts[:, :, 2].sum())
                # SpMV after the scrub: clean matrix -> no further detections (single) / DUEs again (double)
                spmv_det = None
                if check_spmv:
                    c2 = abft.Counters()
                    y = abft.Vector.empty(N, S)
                    abft.spmv(ctx, A, vecs[3], y, c2)
                    spmv_det = int(c2.read()[:, :, 0].sum())
                results.append({"kind": kind, "rate": rate, "seed": seed, "flips": int(k), "codewords": len(touched),
                                "detected": det, "corrected": cor, "uncorrectable": unc, "oracle_match": ok,
                                "spmv_detections_after_scrub": spmv_det, "seconds": round(time.time() - t0, 2)})
                print(json.dumps(results[-1]), flush=True)
    summary = {"grid": grid, "words": words, "trials": len(results),
               "all_match_oracle": all(r["oracle_match"] for r in results),
               "single_flip_codewords": sum(r["codewords"] for r in results if r["kind"] == "single"),
               "single_corrected": sum(r["corrected"] for r in results if r["kind"] == "single"),
               "single_uncorrectable": sum(r["uncorrectable"] for r in results if r["kind"] == "single"),
               "double_uncorrectable": sum(r["uncorrectable"] for r in results if r["kind"] == "double"),
               "double_codewords": sum(r["codewords"] for r in results if r["kind"] == "double")}
    if out_path:
        os.makedirs(os.path.dirname(out_path) or ".", exist_ok=True)
        json.dump({"summary": summary, "trials": results}, open(out_path, "w"), indent=1)
    print(json.dumps(summary))
    return summary, results


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--grid", type=int, default=4096)
    ap.add_argument("--rates", default="1e-9,1e-8,1e-7,1e-6,1e-5")
    ap.add_argument("--seeds", type=int, default=20)
    ap.add_argument("--kind", default="both", choices=["single", "double", "both"])
    ap.add_argument("--out", default=os.path.join(ROOT, "gpurun_out", "campaign.json"))
    a = ap.parse_args()
    kinds = ["single", "double"] if a.kind == "both" else [a.kind]
    run(a.grid, [float(x) for x in a.rates.split(",")], a.seeds, kinds, a.out)


if __name__ == "__main__":
    main()
