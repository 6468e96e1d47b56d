/*
 * abft.h — C ABI of libabft.so: the ABFT-protected CG hot path on B200 (sm_100a).
 *
 * The calls follow the paper's statement of the problem (Pawelczak et al.,
 * CLUSTER 2017; P:a-b = /root/reference/PAPER.md lines):
 *   protect a CSR matrix (val, col, rowptr) and dense fp64 vectors with
 *   SED / SECDED64 / SECDED128 / CRC32C at zero storage overhead
 *   (P:146-152); correct single flips and detect double
 *   flips on load; let the application decide on a DUE;
 *   run the protected SpMV and the protected CG (§V-A).
 * The codes themselves are specified in DESIGN.md §3.
 *
 * Conventions
 *  - Every large buffer is DEVICE memory allocated and owned by the caller; the
 *    library never frees it.  Scratch (reduction partials, CG scalars) belongs
 *    to an abft_ctx and is freed by abft_ctx_destroy.
 *  - `stream` is a cudaStream_t passed as void* (NULL = legacy default stream).
 *    Calls are stream-ordered and asynchronous unless documented "syncs".
 *  - Errors are returned as abft_status codes (never exceptions);
 *    abft_last_error() gives a thread-local message for the last non-OK return.
 *  - Host-side metadata (sizes, schemes) is unprotected.
 *  - Handles are not thread-safe.
 */
#ifndef ABFT_H_
#define ABFT_H_
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

/* Protection schemes. */
typedef enum { ABFT_NONE = 0, ABFT_SED = 1, ABFT_SECDED64 = 2, ABFT_SECDED128 = 3, ABFT_CRC32C = 4,
               ABFT_SCHEME_COUNT = 5 } abft_scheme;
/* Counter targets: CSR elements, row pointers, dense vectors. */
typedef enum { ABFT_T_ELEM = 0, ABFT_T_ROWPTR = 1, ABFT_T_VEC = 2, ABFT_T_COUNT = 3 } abft_target;

/* Per (target, scheme) fault counters.  A counters buffer is a
 * DEVICE array abft_counts[ABFT_T_COUNT][ABFT_SCHEME_COUNT] (480 bytes). */
typedef struct { uint64_t detected, corrected, uncorrectable, range_violations; } abft_counts;

typedef enum {
  ABFT_OK = 0,
  ABFT_E_INVALID = -1,        /* bad argument (null pointer, size, scheme, aliasing) */
  ABFT_E_RANGE = -2,          /* an index / nnz exceeds the scheme's capacity */
  ABFT_E_SHAPE = -3,          /* e.g. a CRC32C row with < 4 entries */
  ABFT_E_DUE = -4,            /* uncorrectable error seen under policy abort */
  ABFT_E_NOT_CONVERGED = -5,  /* CG hit max_iters */
  ABFT_E_CUDA = -6,
  ABFT_E_NCCL = -7
} abft_status;

/* One CSR matrix (or one row-block chunk of a larger matrix, reading R7).
 * val: f64[nnz] (never modified except by scrubbing), col: u32[nnz] (ECC in
 * its top bits after encode), rowptr: u32[abft_rowptr_padded_len(nrows, rowptr_scheme)].
 * Local row i writes out[row_base + i]; local column c reads in[col_base + c].
 * stencil_n: performance hint only (row stride of a 5-point stencil, 0 = none);
 * results never depend on it. */
typedef struct {
  int64_t nrows, ncols, nnz;
  int64_t row_base, col_base;
  double* val;
  uint32_t* col;
  uint32_t* rowptr;
  int32_t elem_scheme, rowptr_scheme;
  int64_t stencil_n;
} abft_csr;

/* A dense fp64 vector of logical length n; data has abft_vec_padded_len(n, scheme)
 * entries (padding holds encoded +0.0). */
typedef struct { int64_t n; double* data; int32_t scheme; } abft_vec;

typedef struct abft_ctx abft_ctx;

/* Create / destroy a context on `device` (owns scratch, events, graphs). */
int abft_ctx_create(int device, abft_ctx** out);
int abft_ctx_destroy(abft_ctx* ctx);
/* Fused calc_p (opt-in, default off): when every chunk is on the tiled
 * stencil path, the vector scheme has group size 1 (NONE / SED / SECDED64) and
 * the solve is single-GPU, abft_cg_solve computes calc_p of iteration k
 * (p = enc(fma(beta, p, r))) inside the SpMV of iteration k+1:
 * bit-identical iterates, counters and statuses, 8 fewer bytes per row per
 * iteration.  The context then owns a second p buffer (padded length of p).
 * enable = 0 runs the unfused sequence. */
int abft_ctx_set_fused_cg(abft_ctx* ctx, int enable);
/* CRC32C correction capability of every later call on ctx (reading
 * R9b): bits = 1 (default) 1EC4ED — a failing CRC32C codeword is corrected when
 * one stored bit explains it, 2..4 flips are DUEs; bits = 2 2EC3ED — also the
 * unique stored-bit pair (cold path, O(M^2) syndrome search), 3 flips are DUEs.
 * Only within CRC32C's HD-6 length (message + 32 <= 5243 bits).  Errors:
 * ABFT_E_INVALID (bits not 1 or 2). */
int abft_ctx_set_crc_correction(abft_ctx* ctx, int bits);
/* Programmatic dependent launch between the kernels of abft_cg_solve's
 * iterations (library default off, single GPU): each kernel issues its
 * loads of data the previous kernel does not write (the matrix, vectors from
 * two kernels back) before waiting on it, hiding launch gaps and tails.
 * Results are identical either way. */
int abft_ctx_set_pdl(abft_ctx* ctx, int enable);

int64_t abft_rowptr_padded_len(int64_t nrows, int32_t scheme);  /* pad with copies of nnz (R6) */
int64_t abft_vec_padded_len(int64_t n, int32_t scheme);         /* pad with encoded +0.0 */

/* a0: encode a CSR matrix in place: ECC into col's top bits and rowptr's top bits
 * (P:361-397), validates capacities (ABFT_E_RANGE) and CRC row lengths
 * (ABFT_E_SHAPE).  Syncs `stream` (returns the validation result). */
int abft_csr_encode(abft_ctx* ctx, abft_csr* A, void* stream);

/* a1: encode a vector in place: round_k then ECC in the k low mantissa bits
 * (DESIGN.md §3.6).  Input: plain f64 values in data[0..n). */
int abft_vec_encode(abft_ctx* ctx, abft_vec* v, void* stream);

/* Check every codeword of v, write the masked values to out_masked (device
 * f64[n], may be NULL), count into dcnt (device, may be NULL), scrub single
 * flips in place.  The vector read of PAPER.md P:441-451 (§VI: the reserved
 * low mantissa bits are masked to 0 when the value is used) as a standalone
 * call; checks and counts follow DESIGN.md §3.6 / §3.8. */
int abft_vec_decode(abft_ctx* ctx, abft_vec* v, double* out_masked, abft_counts* dcnt, void* stream);

/* a3: protected SpMV out = A*in over nchunks chunks.
 * dot_out (device f64, may be NULL) receives sum_i in[row]*out[row] over the
 * chunks' rows, RED-1 order.  in and out must not alias. */
int abft_spmv(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* in, abft_vec* out, double* dot_out,
              abft_counts* dcnt, void* stream);

/* Matrix check mode of one SpMV access ("less frequent correctness checking",
 * P:398-425): */
typedef enum {
  ABFT_CHECK_CORRECT = 0,  /* check every element / rowptr group, correct + scrub single flips (default) */
  ABFT_CHECK_DETECT = 1,   /* check, detection only: any failing codeword is a DUE, never scrubbed */
  ABFT_CHECK_RANGE = 2     /* no ECC check: stored bits masked + range checks only */
} abft_check_mode;
/* abft_spmv with an explicit matrix check mode (vectors are always checked). */
int abft_spmv_ex(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* in, abft_vec* out, double* dot_out,
                 abft_counts* dcnt, int32_t check_mode, void* stream);

/* a3 alone, for timing the dominant kernel: the CG iteration's SpMV kernel
 * instantiation (the p.w partial of every reduction block written to the
 * context's scratch) with NO dot reduction launched after it.
 * Same arguments, checks and counters as abft_spmv; the partials are not
 * returned.  bench.py times back-to-back launches of it (roofline). */
int abft_spmv_partials(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* in, abft_vec* out,
                       abft_counts* dcnt, void* stream);

typedef struct {
  double tol;          /* stop when sqrt(r.r) <= tol*sqrt(r0.r0) (R15) */
  int32_t max_iters;
  int32_t due_policy;  /* 0 = abort (finish the iteration, return ABFT_E_DUE), 1 = continue */
  int32_t poll_every;  /* iterations between host polls of the stop flag (0 = default 16) */
  /* check_interval N: 0/1 = check + correct the
   * matrix on every access; N > 1 = matrix access a (init SpMV = 0, iteration
   * k's SpMV = k) is checked for detection only iff a % N == 0 and only
   * range-checked otherwise, plus a detection-only check of the whole matrix
   * after the solve when N does not divide the iteration count (a DUE found
   * there returns ABFT_E_DUE under policy abort).  Vectors: every access. */
  int32_t check_interval;
} abft_cg_opts;

typedef struct { int32_t iters; int32_t status; double rr0, rrn; } abft_cg_result;

/* a2-a7: protected CG.  x holds x0 on entry and the solution on
 * return; r, p, w are work vectors of the same length/scheme.  The iteration
 * runs on the device (alpha/beta/convergence computed by the reduction
 * kernels); the host only polls a stop flag every opts->poll_every
 * iterations.  Syncs `stream`.  Returns res->status. */
int abft_cg_solve(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                  abft_vec* w, const abft_cg_opts* opts, abft_cg_result* res, abft_counts* dcnt, void* stream);

/* Single-reduction protected CG (S§8(f) f3, reading R28): the
 * Chronopoulos-Gear recurrences — per iteration one fused update
 * (p = r + beta p, s = w + beta s, x += alpha p, r -= alpha s; every operand
 * checked, every result re-encoded) and one protected SpMV w = A r
 * carrying BOTH dot products (r.r, w.r) into ONE reduction, instead of two.
 * Same matrix / vector conventions, options, counters and statuses as
 * abft_cg_solve; s is a sixth vector like the others (scheme, length).
 * Single GPU, every access checked (check_interval <= 1, else ABFT_E_SHAPE). */
/* Protected Chebyshev iteration (S§8(f) f4: TeaLeaf's Chebyshev solver,
 * ref [19] P:778-781, reading R32) for an SPD matrix with
 * spectrum inside [eigmin, eigmax]: per step one protected SpMV w = A u and one
 * fused update r = b - w, p = alpha_k p + beta_k r (first step p = r/theta),
 * u += p with r.r, every operand checked and every result re-encoded as in the
 * paper's CG.  x holds u (in: u0, out: u); stops when
 * sqrt(r.r) <= tol sqrt(r0.r0).  Same conventions, counters and statuses as
 * abft_cg_solve; single GPU, every access checked.  Errors: ABFT_E_INVALID
 * (eigmax <= eigmin), ABFT_E_SHAPE. */
int abft_cheby_solve(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                     abft_vec* w, double eigmin, double eigmax, const abft_cg_opts* opts, abft_cg_result* res,
                     abft_counts* dcnt, void* stream);
/* Protected PPCG (S§8(f) f4: TeaLeaf's polynomially preconditioned CG;
 * DESIGN.md §4.4, reading R34): CG whose preconditioner z = M^-1 r is `inner`
 * (1..64) Chebyshev steps (as abft_cheby_solve's, bounds [eigmin, eigmax]) on
 * A z = r from z = 0; beta = (r.z)'/(r.z), p = z + beta p.  z, rin, pin are
 * three more vectors like the others (the preconditioner's iterate, residual
 * and direction).  Same conventions, counters and statuses as abft_cg_solve;
 * single GPU, every access checked. */
int abft_ppcg_solve(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                    abft_vec* w, abft_vec* z, abft_vec* rin, abft_vec* pin, double eigmin, double eigmax, int inner,
                    const abft_cg_opts* opts, abft_cg_result* res, abft_counts* dcnt, void* stream);
/* TeaLeaf's spectrum estimate (reading R33): `steps` (2..128)
 * protected CG iterations from x (opts supply the policy; tol is ignored),
 * then the extreme eigenvalues of the Lanczos tridiagonal built from the CG
 * step coefficients (T_jj = 1/alpha_j + beta_{j-1}/alpha_{j-1},
 * T_{j,j+1} = sqrt(beta_j)/alpha_j) by Sturm bisection.  x is left at the CG
 * iterate.  The caller applies any safety margin. */
int abft_cg_spectrum(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                     abft_vec* w, int steps, const abft_cg_opts* opts, double* eigmin, double* eigmax,
                     abft_cg_result* res, abft_counts* dcnt, void* stream);
int abft_cg_solve_sr(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r,
                     abft_vec* p, abft_vec* w, abft_vec* s, const abft_cg_opts* opts, abft_cg_result* res,
                     abft_counts* dcnt, void* stream);

/* a4 / a5 as single calls (the CG driver fuses them into its device-side loop):
 * calc_ur  x = enc(fma(alpha, p, x)); r = enc(fma(-alpha, w, r)); rrn_out = r.r (RED-1)
 * calc_p   p = enc(fma(beta, p, r))
 * (TeaLeaf CG).  Every operand codeword is checked on
 * load and single flips corrected (counted into dcnt, may be NULL); x, r, p, w
 * must have equal length and scheme and must not alias.  rrn_out: device f64
 * (may be NULL). */
int abft_calc_ur(abft_ctx* ctx, abft_vec* x, abft_vec* p, abft_vec* r, abft_vec* w, double alpha, double* rrn_out,
                 abft_counts* dcnt, void* stream);
int abft_calc_p(abft_ctx* ctx, abft_vec* p, abft_vec* r, double beta, abft_counts* dcnt, void* stream);

/* a5 + a3 fused: p_out = enc(fma(beta, p_prev, r)) (calc_p,
 * P:294-314) and out = A*p_out (+ dot_out = p_out.out, RED-1) in ONE tiled
 * kernel — the same words and counters as abft_calc_p(p_prev, r, beta)
 * followed by abft_spmv(p_prev, out), except that p_prev itself is left as
 * it was (single flips scrubbed) and the new p goes to p_out.  Requires the
 * tiled stencil path (stencil_n) for every chunk and a group-size-1 vector
 * scheme (NONE / SED / SECDED64), else ABFT_E_SHAPE.  p_prev, r, p_out, out:
 * equal length and scheme, pairwise distinct. */
int abft_calc_p_spmv(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* p_prev, abft_vec* r, double beta,
                     abft_vec* p_out, abft_vec* out, double* dot_out, abft_counts* dcnt, void* stream);

/* Check every codeword of the matrix chunks and of the nvec vectors, counting
 * into dcnt.  scrub: 0 count only, 1 count and correct single flips in place,
 * 2 detection only (every failing codeword is a DUE, nothing is written).
 * The whole-structure check of PAPER.md P:398-425 (§VI "less frequent
 * correctness checking": the full check at the end of a solve whose
 * interval does not divide the iteration count) and the config-5 campaign's
 * per-trial check (SURVEY S§8(d)); semantics DESIGN.md §3.8 / §3.9. */
int abft_check_all(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* vecs, int nvec, int scrub,
                   abft_counts* dcnt, void* stream);

/* Fault injection (not in the paper; the harness of S§3.4): XOR one stored bit
 * at bit_offset of the device buffer dev_base.  Stream-ordered. */
int abft_inject_bitflip(abft_ctx* ctx, void* dev_base, uint64_t bit_offset, void* stream);
/* Scheduled fault injection (S§8(c) O10, the harness of BASELINE configs 1 and
 * 5): fault i XORs bit `bit` of storage word `word` of `target` — matrix chunk
 * `chunk`'s val (64-bit words), col or rowptr (32-bit words), or the CG vector
 * b, x, r, p, w (64-bit words, vecs[target - ABFT_F_B]) — before init (iter 0)
 * or before iteration `iter`'s SpMV, inside the solve (a device-side kernel
 * reads the iteration counter, so CUDA-graph replays apply it too).  The
 * schedule (device copy owned by ctx) applies to every later abft_cg_solve /
 * abft_cg_solve_dist on ctx with the SAME matrix and vector buffers, until
 * replaced; nfaults = 0 clears it.  A schedule turns the fused calc_p off.
 * Errors: ABFT_E_INVALID (bad target / chunk / word / bit), ABFT_E_CUDA. */
typedef enum { ABFT_F_VAL = 0, ABFT_F_COL = 1, ABFT_F_ROWPTR = 2, ABFT_F_B = 3, ABFT_F_X = 4, ABFT_F_R = 5,
               ABFT_F_P = 6, ABFT_F_W = 7 } abft_fault_target;
typedef struct { int32_t iter; int32_t target; int64_t word; int32_t bit; int32_t chunk; } abft_fault;
int abft_ctx_set_faults(abft_ctx* ctx, const abft_fault* faults, int nfaults, const abft_csr* A, int nchunks,
                        abft_vec* const* vecs /* [5]: b, x, r, p, w */);

/* Copy the device counters to host_out[ABFT_T_COUNT*ABFT_SCHEME_COUNT].  Syncs.
 * The per-scheme detected / corrected / uncorrectable counts the paper's
 * evaluation reports (§VII) and north_star asks for;
 * counting rule DESIGN.md §3.8 (first logical read, owner counts). */
int abft_counts_read(const abft_counts* dcnt, abft_counts* host_out, void* stream);
int abft_counts_reset(abft_counts* dcnt, void* stream);

/* Number of kernels this process launched through the library so far. */
uint64_t abft_launch_count(void);

/* Per-kernel-class device time accumulated by the CG driver when profiling is
 * on (CUDA events on the launch stream): class 0 SpMV, 1 calc_ur, 2 calc_p,
 * 3 reductions.  abft_profile(ctx, 1) clears and enables. */
int abft_profile(abft_ctx* ctx, int enable);
int abft_profile_read(abft_ctx* ctx, double* ms_out /*[4]*/, int64_t* launches_out /*[4]*/);

const char* abft_last_error(void);

/* ---- multi-GPU (row-block strips, reading S§8(e)) ----
 * One process per GPU.  nccl_unique_id: 128 bytes from ncclGetUniqueId on rank 0,
 * broadcast by the caller (torch.distributed).  The local vectors have n_halo
 * extra entries before and after the local rows (ghost rows of the strip). */
typedef struct abft_dist abft_dist;
int abft_dist_init(abft_dist** out, const void* nccl_unique_id, int rank, int nranks, int device);
int abft_dist_get_unique_id(void* out128);
int abft_dist_destroy(abft_dist* d);
/* Distributed protected CG: each rank passes its strip's chunks (col_base
 * relative to the halo-extended vector) and its halo-extended vectors; halos of
 * encoded p are exchanged with rank-1 / rank+1 before each SpMV, and the RED-1
 * subtree roots of the two dot products are all-gathered (bit-identical to one
 * GPU when every rank owns a power-of-two number of reduction blocks). */
int abft_cg_solve_dist(abft_dist* d, abft_ctx* ctx, const abft_csr* A, int nchunks, int64_t n_halo, abft_vec* b,
                       abft_vec* x, abft_vec* r, abft_vec* p, abft_vec* w, const abft_cg_opts* opts,
                       abft_cg_result* res, abft_counts* dcnt, void* stream);
/* In-process LOOPBACK transport (testing the P > 1 path on one device): nranks
 * virtual ranks whose strips all live in this process on `device`.  The halo
 * step becomes device-to-device copies between the ranks' extended vectors and
 * the all-gather a shared device buffer; every other step (kernels, RED-1
 * subtree roots, top-of-tree combine, DUE consensus, interior/boundary split,
 * CUDA graph) is the code the NCCL transport runs.  Errors: ABFT_E_INVALID
 * (nranks < 1 or > 1024), ABFT_E_CUDA. */
int abft_dist_init_loopback(abft_dist** out, int nranks, int device);

/* Peer-memory halos (SURVEY S§8(f) f3 "NVLink P2P / symmetric-memory halos";
 * the halo exchange of PAPER.md P:300-301 §V-A's decomposed grid done by the
 * producer of p): with enable = 1 the standard CG's calc_p also stores the
 * encoded p of its first / last local grid row straight into the neighbours'
 * ghost rows, k_post_p then raises the neighbours' arrival flags
 * (system-scope fence + atomic store of the iteration count), and each SpMV's
 * halo step becomes a one-thread wait on this rank's two flags (on the comm
 * stream, overlapped with the interior tile rows).  Iteration 1 still copies
 * the init p once.  Same words, counters and results as the copy exchange.
 * Used only for the standard CG with equal strips and no fault schedule;
 * otherwise the copy exchange runs.
 *   loopback transport: peer_p / peer_flag ignored (the ranks' own buffers).
 *   NCCL transport: peer_p[0] / peer_p[1] = rank-1's / rank+1's halo-extended
 *   p data mapped into this process (abft_ipc_open_handle; NULL where there is
 *   no neighbour), peer_flag[0] = rank-1's flags + 1, peer_flag[1] = rank+1's
 *   flags + 0 (abft_dist_flags of the neighbour, mapped).  The buffers must
 *   stay valid for the solves that use them.
 * enable = 0 restores the copy exchange.  ABFT_E_INVALID on missing pointers. */
int abft_dist_set_peer_halo(abft_dist* d, int enable, void* const* peer_p, int* const* peer_flag);
/* This rank's two arrival-flag words (device memory of the transport; [0] is
 * raised by rank-1, [1] by rank+1) — to be shared with the neighbours. */
int abft_dist_flags(abft_dist* d, int** flags);
/* CUDA IPC for the NCCL transport's peer halos: the 64-byte handle of the
 * allocation holding dev_ptr and dev_ptr's offset in it; open maps a peer's
 * handle (+ offset) into this process (peer access enabled lazily); close
 * unmaps (pass the same offset). */
int abft_ipc_get_handle(const void* dev_ptr, void* handle64, int64_t* offset);
int abft_ipc_open_handle(const void* handle64, int64_t offset, void** dev_ptr);
int abft_ipc_close_handle(void* dev_ptr, int64_t offset);
/* Distributed protected CG over a loopback transport: per rank q, ctxs[q] (one
 * context per rank, all on the transport's device), its chunk array A[q] of
 * nchunks[q] chunks, its halo-extended vectors vecs[5q .. 5q+4] = b, x, r, p, w,
 * its counters dcnt[q] and its result res[q].  All ranks run in lockstep on
 * `stream`; the return value is rank 0's status.  Same semantics and results as
 * abft_cg_solve_dist on nranks processes (S§8(e), §V-A). */
int abft_cg_solve_loopback(abft_dist* d, abft_ctx* const* ctxs, const abft_csr* const* A, const int* nchunks,
                           int64_t n_halo, abft_vec* const* vecs, const abft_cg_opts* opts, abft_cg_result* res,
                           abft_counts* const* dcnt, void* stream);
/* Single-reduction CG on row-block strips (S§8(e) + f3): the halo exchanged
 * before each SpMV is r's (the SpMV's input), and the ONE all-gather per
 * iteration carries (w.r root, DUE flag, r.r root) per rank.  Same strip
 * conventions as abft_cg_solve_dist / abft_cg_solve_loopback; the loopback
 * variant takes vecs[6q .. 6q+5] = b, x, r, p, w, s per rank. */
int abft_cg_solve_sr_dist(abft_dist* d, abft_ctx* ctx, const abft_csr* A, int nchunks, int64_t n_halo, abft_vec* b,
                          abft_vec* x, abft_vec* r, abft_vec* p, abft_vec* w, abft_vec* s, const abft_cg_opts* opts,
                          abft_cg_result* res, abft_counts* dcnt, void* stream);
int abft_cg_solve_loopback_sr(abft_dist* d, abft_ctx* const* ctxs, const abft_csr* const* A, const int* nchunks,
                              int64_t n_halo, abft_vec* const* vecs, const abft_cg_opts* opts, abft_cg_result* res,
                              abft_counts* const* dcnt, void* stream);


/* Host-side codec hooks (no GPU needed): run the exact __host__ __device__
 * codec functions on the CPU for the unit tests.  inst: 0 E-SECDED, 1 V-SECDED64,
 * 2 R-SECDED64, 3 R-SECDED128, 4 V-SECDED128.  Returns 0 clean, 1 corrected, 2 DUE.
 * inst 5 / 6 (check only): the tiled SpMV's pair-packed fast checks of two
 * E-SECDED codewords words[0..2], words[3..5] / two V-SECDED64 codewords
 * words[0..1], words[2..3]: 0 iff both are clean, else 2. */
int abft_codec_host_check(int inst, uint32_t* words);
void abft_codec_host_encode(int inst, uint32_t* words);

#ifdef __cplusplus
}
#endif
#endif /* ABFT_H_ */
