// internal.h — host-side interface between the C ABI (capi.cu, dist.cu) and the
// kernel translation unit (kernels.cu).  No torch types anywhere.
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include "../../include/abft.h"

namespace abft {

// Device CG scalars.  Written only by single threads of the
// reduction kernels' last blocks and by calc_p's last block.
struct CgState {
  double rr0, rro, rrn, pw, alpha, beta, tol;
  int32_t iters, max_iters, stop, status, abort_policy, converged;
  uint32_t ticket_p;   // calc_p last-block ticket
  int32_t dist;        // 1 = multi-GPU solve (abort decided after an all-gather)
  // fused calc_p: calc_p of iteration k runs inside the SpMV
  // of iteration k+1, so the stop decisions calc_p's last block takes move to
  // the rrn reduction; a stop that the unfused order takes AFTER calc_p leaves
  // pending_p = 1 and the host runs that calc_p on its own.
  int32_t fused, pending_p;
  // Chebyshev iteration: theta, delta, sigma of the spectrum
  // bounds and the recurrence's rho (alpha / beta above hold its step
  // coefficients)
  double ch_theta, ch_delta, ch_sigma, ch_rho;
  int32_t pcg;   // PPCG: rro holds r.z, kept by k_post_p
  // CG step coefficients of the first CG_LOG iterations (Lanczos data of the
  // spectrum estimate, abft_cg_spectrum): ctx-owned device arrays [CG_LOG]
  double* alpha_log;
  double* beta_log;
};
constexpr int CG_LOG = 128;
// multi-rank all-gather payload per rank: (RED-1 subtree root, DUE flag,
// second root — the single-reduction CG's r.r)
constexpr int GATHER_W = 3;

struct DevCounts { unsigned long long v[3][5][4]; };

// One scheduled fault (S§8(c) O10) resolved to a device word: XOR `mask` into
// the 32-bit word at `addr` before iteration `iter`'s SpMV (0 = before init).
struct DevFault { uint32_t* addr; uint32_t mask; int32_t iter; };

// CRC32C lookup tables (reflected 0x82F63B78), built once per
// context on the host and copied to shared memory by the kernels that use them.
struct CrcTables {
  uint32_t slice[4][256];     // slicing-by-4: slice[k][b] = CRC register of byte b followed by k zero bytes
  uint32_t vpos[4][7][256];   // V-CRC: linear CRC part of byte b at message byte 8t + j + 1 of the 32-byte quad
};
void build_crc_tables(CrcTables* host_out);

// arguments of one SpMV chunk launch
struct SpmvArgs {
  int64_t nrows, ncols, nnz, row_base, col_base, n_in, npad_in, npad_out, rb_offset;
  int64_t stencil_n;  // > 0: 5-point stencil row stride (tiled fast path)
  // tiled path only: launch the tile rows [ty_lo, ty_hi) of the chunk (ty_hi =
  // 0: all) — the interior / boundary split that overlaps the halo exchange
  int64_t ty_lo, ty_hi;
  uint64_t* val;
  uint32_t* col;
  uint32_t* rowptr;
  uint64_t* in;
  uint64_t* out;
  double* partials;  // indexed rb_offset + local RB (may be null)
  double* partials2; // DOT 2 (single-reduction CG): in.in partials, same indexing
  DevCounts* counts; // may be null
  int* due;          // DUE / range flag (never null)
  const CgState* state;  // may be null
  // matrix check mode of this access: MODE_CORRECT / DETECT /
  // RANGE; with check_interval > 1 the kernel derives it from the device
  // iteration counter instead (access k = state->iters + 1, init = 0)
  int32_t check_mode, check_interval;
  const CrcTables* crc;   // device tables (CRC32C schemes only)
  // fused calc_p (CG driver only, tiled path, G = 1 vector schemes,
  // DESIGN.md §6.1): p is double-buffered.  Iteration k >= 2 reads
  // p_{k-1} from `in` and r from r_f, computes p_k = enc(round(fma(beta,
  // p_{k-1}, r))) into p_cur and multiplies by it; iteration 1 (state->iters
  // == 0) multiplies by p_1 = p_cur as written by init.  The buffer roles
  // alternate with the parity of k (host side).  fz / beta_f are filled in by
  // the kernel (SMEM copy of the arguments).
  uint64_t* p_cur;
  uint64_t* r_f;
  double beta_f;
  int32_t fz;
  // 1: no kernel between the one that last wrote `in` and this SpMV's direct
  // predecessor writes `in` (the CG loop's SpMV of p after calc_p + k_post_p,
  // no fault schedule), so the tiled kernel may issue its `in` window TMA
  // before the PDL wait
  int32_t early_in;
};
enum { MODE_CORRECT = 0, MODE_DETECT = 1, MODE_RANGE = 2 };

struct VecArgs {
  int64_t n, npad;
  uint64_t* x; uint64_t* p; uint64_t* r; uint64_t* w; uint64_t* b;
  double* partials;
  DevCounts* counts;
  int* due;
  CgState* state;
  double* out_masked;
  const CrcTables* crc;   // device tables (CRC32C schemes only)
  // peer-memory halos (multi-rank): calc_p also stores the
  // encoded p of its first / last halo_n local rows straight into the
  // neighbours' ghost rows (halo_up: rank-1's bottom ghost row, halo_dn:
  // rank+1's top ghost row; null = no such neighbour), and k_post_p then raises
  // the neighbours' arrival flags (sig_up / sig_dn) to the iteration count
  uint64_t* halo_up;
  uint64_t* halo_dn;
  int64_t halo_n;
  int* sig_up;
  int* sig_dn;
};

// PDL for the CG driver's iteration launches
void set_pdl(bool on);
// write the device CG state from a by-value launch argument (no host staging buffer)
int launch_set_state(const CgState& h, CgState* dst, cudaStream_t s);
// launchers (kernels.cu); each returns the number of kernels launched
// dot: 0 none, 1 in.out -> partials, 2 also in.in -> partials2
int launch_spmv(const SpmvArgs& a, int es, int rs, int vs, int dot, cudaStream_t s);
// -1: a fused-calc_p launch (a.p_cur set) could not run
// can this chunk take the fused-calc_p tiled SpMV (G = 1 vector scheme, stencil layout)?
bool spmv_fusable(const SpmvArgs& a, int vs);
// will this chunk run on the tiled stencil kernel (so a tile-row split is possible)?
bool spmv_tileable(const SpmvArgs& a, int vs);
int64_t spmv_tile_rows(const SpmvArgs& a);   // tile rows of a tileable chunk
int launch_calc_ur(const VecArgs& a, int vs, cudaStream_t s);
int launch_calc_p(const VecArgs& a, int vs, cudaStream_t s);
int launch_init_r(const VecArgs& a, int vs, cudaStream_t s);
int launch_vec_encode(uint64_t* data, int64_t n, int64_t npad, int vs, cudaStream_t s);
int launch_vec_check(uint64_t* data, int64_t n, int64_t npad, int vs, double* out_masked, DevCounts* c, int* due,
                     int scrub, cudaStream_t s);
// op: 0 plain dot -> *out, 1 rr0 (init), 2 pw (alpha), 3 rrn (convergence, beta),
//     4 subtree root + DUE flag -> out[0..2) (multi-GPU all-gather payload)
int launch_reduce(const double* partials, int64_t nrb, double* roots, uint32_t* ticket, int op, CgState* st,
                  double* out, const int* due, cudaStream_t s);
// single-reduction CG: reduce partials (w.r) and partials2
// (r.r) in RED-1 order and apply op 7 (init) / 6 (iteration)
int launch_reduce_sr(const double* partials, const double* partials2, int64_t nrb, double* roots, double* roots2,
                     uint32_t* ticket, int op, CgState* st, const int* due, cudaStream_t s);
// Chebyshev update (DESIGN.md §4.3 / §4.4).  mode: 0 step, 1 first step (p =
// r/theta), coefficients from the CG state; 2 step, 3 first step from u = 0
// (no w, no u read), coefficients alpha / beta / theta as given (the PPCG
// preconditioner's inner steps).
int launch_cheb(const VecArgs& a, int vs, int mode, double alpha, double beta, double theta, cudaStream_t s);
// checked dot a.r . a.x (RED-1 partials; PPCG's r.z)
int launch_dot(const VecArgs& a, int vs, cudaStream_t s);
// dst = src (encoded words, npad entries) unless the solve stopped
int launch_copy_running(uint64_t* dst, const uint64_t* src, int64_t npad, const CgState* st, cudaStream_t s);
// single-reduction CG update: p, s, x, r (VecArgs.b carries s)
int launch_calc_sr(const VecArgs& a, int vs, cudaStream_t s);
// single-reduction CG, multi-rank: op 10 -> out[0..3) = (w.r root, DUE flag, r.r root)
int launch_reduce_sr_root(const double* partials, const double* partials2, int64_t nrb, double* roots, double* roots2,
                          uint32_t* ticket, double* out, const int* due, cudaStream_t s);
int launch_combine_sr(const double* gathered, int P, int op, CgState* st, int* due, cudaStream_t s);
int launch_combine(const double* gathered, int P, int op, CgState* st, int* due, cudaStream_t s);
int launch_due_combine(const double* gathered, int P, CgState* st, int* due, cudaStream_t s);
int launch_pack_due(double* out, const int* due, cudaStream_t s);
int launch_csr_encode(abft_csr* A, uint32_t* flags, cudaStream_t s);
int launch_check_csr(const abft_csr* A, DevCounts* c, int* due, int scrub, cudaStream_t s);
int launch_inject(void* base, uint64_t bit, cudaStream_t s);
int launch_wait_halo(const int* flags, const CgState* st, int need_up, int need_dn, cudaStream_t s);
void prepare_kernels(int device);
// phase 0: the faults of iteration 0 (before init); phase 1: those of
// iteration state->iters + 1 (skipped once the solve stopped)
int launch_inject_sched(const DevFault* f, int n, const CgState* st, int phase, cudaStream_t s);

int64_t rowptr_padded_len(int64_t nrows, int scheme);
int64_t vec_padded_len(int64_t n, int scheme);

}  // namespace abft
