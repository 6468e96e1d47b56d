// kernels.cu — every device kernel of the ABFT-protected CG hot path (sm_100a).
//
// Scope rows (DESIGN.md §1 / SURVEY §8(a)):
//   a0 k_encode_elems / k_encode_rowptr / k_encode_ecrc   CSR encode
//   a1 k_vec_encode                                        vector encode
//   a2 k_init_r                                            r = b - A x0, p = r, rr0
//   a3 k_spmv                                              protected SpMV + p.w
//   a4 k_calc_ur                                           x += a p, r -= a w, r.r
//   a5 k_calc_p                                            p = r + b p
//   a6 k_reduce                                            RED-1 tree + alpha/beta/convergence
//   a7 counters / DUE policy / k_check_* / k_inject
//
// Work decomposition (all BLAS-1 and the SpMV): one warp per reduction block
// (RB) of 256 consecutive rows, processed as 8 passes of 32 rows — lane l
// handles rows l, l+32, ..., l+224 of its RB, which IS the RED-1 order of
// DESIGN.md §4, so the fused dot products need no reordering.  Each pass
// issues fully coalesced 8-byte loads of the vectors (one 256-byte line per
// warp-instruction).  The codec fast path ("is this codeword clean?") is
// inline; locating/correcting a flip is a __noinline__ cold path.
#include <atomic>

#include "kernels_impl.cuh"

namespace abft {

thread_local bool g_pdl = false;
void set_pdl(bool on) { g_pdl = on; }

// CG scalars written by a kernel (arguments captured at launch), never by an
// async copy of a host buffer that a later call could overwrite first.
static __global__ void k_set_state(CgState h, CgState* dst) { *dst = h; }
int launch_set_state(const CgState& h, CgState* dst, cudaStream_t s) {
  k_set_state<<<1, 1, 0, s>>>(h, dst);
  return 1;
}

// per-ES SpMV launchers live in spmv_es*.cu (parallel compilation)
bool spmv_es_none(const SpmvArgs&, int, int, int, cudaStream_t);
bool spmv_es_sed(const SpmvArgs&, int, int, int, cudaStream_t);
bool spmv_es_secded(const SpmvArgs&, int, int, int, cudaStream_t);
bool spmv_es_crc(const SpmvArgs&, int, int, int, cudaStream_t);

int launch_spmv(const SpmvArgs& a, int es, int rs, int vs, int dot, cudaStream_t s) {
  if (a.nrows <= 0) return 0;
  bool ok;
  switch (es) {
    case NONE: ok = spmv_es_none(a, rs, vs, dot, s); break;
    case SED: ok = spmv_es_sed(a, rs, vs, dot, s); break;
    case SECDED64:
    case SECDED128: ok = spmv_es_secded(a, rs, vs, dot, s); break;  // R3: both map to E-SECDED
    default: ok = spmv_es_crc(a, rs, vs, dot, s); break;
  }
  return ok ? 1 : -1;
}

// ================================================================ launchers
static inline int grid_for(int64_t n, int threads, int max_blocks = 148 * 16) {
  int64_t b = (n + threads - 1) / threads;
  if (b < 1) b = 1;
  if (b > max_blocks) b = max_blocks;
  return (int)b;
}

#define ABFT_VS_DISPATCH(vs, F, ...)                      \
  switch (vs) {                                           \
    case NONE: F<NONE><<<__VA_ARGS__>>>; break;           \
    case SED: F<SED><<<__VA_ARGS__>>>; break;             \
    case SECDED64: F<SECDED64><<<__VA_ARGS__>>>; break;   \
    case SECDED128: F<SECDED128><<<__VA_ARGS__>>>; break; \
    default: F<CRC32C><<<__VA_ARGS__>>>; break;           \
  }

static inline int blocks_rb(int64_t n) { return (int)(((n + 255) / 256 + 7) / 8); }

// CRC32C tables: reflected polynomial 0x82F63B78, bytes LSB first.
void build_crc_tables(CrcTables* T) {
  for (uint32_t b = 0; b < 256; b++) {
    uint32_t c = b;
    for (int k = 0; k < 8; k++) c = (c >> 1) ^ (0x82F63B78u & (0u - (c & 1u)));
    T->slice[0][b] = c;
  }
  for (int k = 1; k < 4; k++)
    for (uint32_t b = 0; b < 256; b++) {
      const uint32_t c = T->slice[k - 1][b];
      T->slice[k][b] = (c >> 8) ^ T->slice[0][c & 0xFFu];
    }
  // linear part of byte b at position p of a 32-byte message: register T0[b]
  // after that byte (init 0), then 31 - p zero bytes
  for (int t = 0; t < 4; t++)
    for (int j = 1; j < 8; j++)
      for (uint32_t b = 0; b < 256; b++) {
        uint32_t c = T->slice[0][b];
        for (int z = 0; z < 31 - (8 * t + j); z++) c = (c >> 8) ^ T->slice[0][c & 0xFFu];
        T->vpos[t][j - 1][b] = c;
      }
}

int launch_calc_ur(const VecArgs& a, int vs, cudaStream_t s) {
  if (a.n <= 0) return 0;
  int nb = blocks_rb(a.n);
  switch (vs) {
    case NONE: launch_k(k_calc_ur<NONE>, nb, 256, 0, s, a); break;
    case SED: launch_k(k_calc_ur<SED>, nb, 256, 0, s, a); break;
    case SECDED64: launch_k(k_calc_ur<SECDED64>, nb, 256, 0, s, a); break;
    case SECDED128: launch_k(k_calc_ur<SECDED128>, nb, 256, 0, s, a); break;
    default: launch_k(k_calc_ur<CRC32C>, nb, 256, vec_dyn_smem<CRC32C>(), s, a); break;
  }
  return 1;
}
// ABFT_P_BULK = 1: G = 1 schemes on whole CP_STAGE-row stages take the
// bulk-copy staged persistent kernel k_calc_p_bulk.  Default 0: measured
// 0.0888 vs 0.0799 ms protected, 0.0747 vs 0.0698 twin (r2r, same box)
#ifndef ABFT_P_BULK
#define ABFT_P_BULK 0
#endif
// per-device function attributes of the kernels with > 48 KB of dynamic SMEM
// that may first launch inside a CG-graph capture (abft_ctx_create calls this)
void prepare_kernels(int device) {
  (void)device;
  cudaFuncSetAttribute(k_calc_p_bulk<NONE>, cudaFuncAttributeMaxDynamicSharedMemorySize, CP_SMEM);
  cudaFuncSetAttribute(k_calc_p_bulk<SED>, cudaFuncAttributeMaxDynamicSharedMemorySize, CP_SMEM);
  cudaFuncSetAttribute(k_calc_p_bulk<SECDED64>, cudaFuncAttributeMaxDynamicSharedMemorySize, CP_SMEM);
}
template <int VS>
static void calc_p_bulk(const VecArgs& a, cudaStream_t s) {
  static std::atomic<int> grid{0};   // CTAs resident at once (persistent grid)
  if (!grid.load(std::memory_order_relaxed)) {
    int dev = 0, sms = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    grid.store(sms * CP_CTAS_PER_SM, std::memory_order_relaxed);
  }
  const int64_t nstage = a.n / CP_STAGE;
  const int gmax = grid.load(std::memory_order_relaxed);
  const int g = (int)(nstage < gmax ? nstage : gmax);
  launch_k(k_calc_p_bulk<VS>, g, 256, CP_SMEM, s, a);
}
int launch_calc_p(const VecArgs& a, int vs, cudaStream_t s) {
  if (a.n <= 0) return 0;
  int nb = blocks_rb(a.n);
  if (ABFT_P_BULK && (a.n % CP_STAGE) == 0 && (vs == NONE || vs == SED || vs == SECDED64)) {
    if (vs == NONE) calc_p_bulk<NONE>(a, s);
    else if (vs == SED) calc_p_bulk<SED>(a, s);
    else calc_p_bulk<SECDED64>(a, s);
    launch_k(k_post_p, 1, 1, 0, s, a.state, (const int*)a.due, a.sig_up, a.sig_dn);
    return 2;
  }
  switch (vs) {
    case NONE: launch_k(k_calc_p<NONE>, nb, 256, 0, s, a); break;
    case SED: launch_k(k_calc_p<SED>, nb, 256, 0, s, a); break;
    case SECDED64: launch_k(k_calc_p<SECDED64>, nb, 256, 0, s, a); break;
    case SECDED128: launch_k(k_calc_p<SECDED128>, nb, 256, 0, s, a); break;
    default: launch_k(k_calc_p<CRC32C>, nb, 256, vec_dyn_smem<CRC32C>(), s, a); break;
  }
#if ABFT_P_TICKET
  return 1;
#else
  launch_k(k_post_p, 1, 1, 0, s, a.state, (const int*)a.due, a.sig_up, a.sig_dn);
  return 2;
#endif
}
int launch_calc_sr(const VecArgs& a, int vs, cudaStream_t s) {
  if (a.n <= 0) return 0;
  int nb = blocks_rb(a.n);
  switch (vs) {
    case NONE: launch_k(k_calc_sr<NONE>, nb, 256, 0, s, a); break;
    case SED: launch_k(k_calc_sr<SED>, nb, 256, 0, s, a); break;
    case SECDED64: launch_k(k_calc_sr<SECDED64>, nb, 256, 0, s, a); break;
    case SECDED128: launch_k(k_calc_sr<SECDED128>, nb, 256, 0, s, a); break;
    default: launch_k(k_calc_sr<CRC32C>, nb, 256, vec_dyn_smem<CRC32C>(), s, a); break;
  }
  return 1;
}
template <int MODE>
static void launch_cheb_t(const VecArgs& a, int vs, double al, double be, double th, cudaStream_t s) {
  int nb = blocks_rb(a.n);
  switch (vs) {
    case NONE: launch_k(k_cheb<NONE, MODE>, nb, 256, 0, s, a, al, be, th); break;
    case SED: launch_k(k_cheb<SED, MODE>, nb, 256, 0, s, a, al, be, th); break;
    case SECDED64: launch_k(k_cheb<SECDED64, MODE>, nb, 256, 0, s, a, al, be, th); break;
    case SECDED128: launch_k(k_cheb<SECDED128, MODE>, nb, 256, 0, s, a, al, be, th); break;
    default: launch_k(k_cheb<CRC32C, MODE>, nb, 256, vec_dyn_smem<CRC32C>(), s, a, al, be, th); break;
  }
}
int launch_cheb(const VecArgs& a, int vs, int mode, double alpha, double beta, double theta, cudaStream_t s) {
  if (a.n <= 0) return 0;
  switch (mode) {
    case 0: launch_cheb_t<0>(a, vs, alpha, beta, theta, s); break;
    case 1: launch_cheb_t<1>(a, vs, alpha, beta, theta, s); break;
    case 2: launch_cheb_t<2>(a, vs, alpha, beta, theta, s); break;
    default: launch_cheb_t<3>(a, vs, alpha, beta, theta, s); break;
  }
  return 1;
}
int launch_dot(const VecArgs& a, int vs, cudaStream_t s) {
  if (a.n <= 0) return 0;
  int nb = blocks_rb(a.n);
  switch (vs) {
    case NONE: launch_k(k_dot<NONE>, nb, 256, 0, s, a); break;
    case SED: launch_k(k_dot<SED>, nb, 256, 0, s, a); break;
    case SECDED64: launch_k(k_dot<SECDED64>, nb, 256, 0, s, a); break;
    case SECDED128: launch_k(k_dot<SECDED128>, nb, 256, 0, s, a); break;
    default: launch_k(k_dot<CRC32C>, nb, 256, vec_dyn_smem<CRC32C>(), s, a); break;
  }
  return 1;
}
int launch_copy_running(uint64_t* dst, const uint64_t* src, int64_t npad, const CgState* st, cudaStream_t s) {
  if (npad <= 0) return 0;
  launch_k(k_copy_running, grid_for(npad, 256), 256, 0, s, dst, src, npad, st);
  return 1;
}
int launch_init_r(const VecArgs& a, int vs, cudaStream_t s) {
  if (a.n <= 0) return 0;
  int nb = blocks_rb(a.n);
  switch (vs) {
    case NONE: k_init_r<NONE><<<nb, 256, 0, s>>>(a); break;
    case SED: k_init_r<SED><<<nb, 256, 0, s>>>(a); break;
    case SECDED64: k_init_r<SECDED64><<<nb, 256, 0, s>>>(a); break;
    case SECDED128: k_init_r<SECDED128><<<nb, 256, 0, s>>>(a); break;
    default: k_init_r<CRC32C><<<nb, 256, 0, s>>>(a); break;
  }
  return 1;
}
int launch_vec_encode(uint64_t* d, int64_t n, int64_t npad, int vs, cudaStream_t s) {
  if (npad <= 0 || vs == NONE) return 0;
  int nb = grid_for(npad, 256);
  switch (vs) {
    case SED: k_vec_encode<SED><<<nb, 256, 0, s>>>(d, n, npad); break;
    case SECDED64: k_vec_encode<SECDED64><<<nb, 256, 0, s>>>(d, n, npad); break;
    case SECDED128: k_vec_encode<SECDED128><<<nb, 256, 0, s>>>(d, n, npad); break;
    default: k_vec_encode<CRC32C><<<nb, 256, 0, s>>>(d, n, npad); break;
  }
  return 1;
}
int launch_vec_check(uint64_t* d, int64_t n, int64_t npad, int vs, double* out, DevCounts* c, int* due, int scrub,
                     cudaStream_t s) {
  if (npad <= 0) return 0;
  int nb = grid_for(npad, 256);
  switch (vs) {
    case NONE: k_vec_check<NONE><<<nb, 256, 0, s>>>(d, n, npad, out, c, due, scrub); break;
    case SED: k_vec_check<SED><<<nb, 256, 0, s>>>(d, n, npad, out, c, due, scrub); break;
    case SECDED64: k_vec_check<SECDED64><<<nb, 256, 0, s>>>(d, n, npad, out, c, due, scrub); break;
    case SECDED128: k_vec_check<SECDED128><<<nb, 256, 0, s>>>(d, n, npad, out, c, due, scrub); break;
    default: k_vec_check<CRC32C><<<nb, 256, 0, s>>>(d, n, npad, out, c, due, scrub); break;
  }
  return 1;
}
// ABFT_RED_CL = 1: the cluster reduction (k_reduce_cl) when the padded leaf
// count allows it.  Default 0 (the multi-block ticket form k_reduce): the
// cluster form measured 9.5 vs 6.3 us per standalone reduction and equal
// inside the PDL CG loop (r2m, same box).
#ifndef ABFT_RED_CL
#define ABFT_RED_CL 0
#endif
template <bool TWO>
static bool launch_reduce_cl(const double* partials, const double* partials2, int64_t nrb, int64_t p2, int op,
                             CgState* st, double* out, const int* due, cudaStream_t s) {
  if (!ABFT_RED_CL || p2 > RED_CL_MAX) return false;
  const int C = p2 >= 4096 ? 8 : (p2 >= 512 ? (int)(p2 / 512) : 1);
  const int64_t L = p2 / C;
  const int lpt = L > 512 ? (int)(L / 512) : 1;
  const int nt = (int)(L / lpt);
  cudaLaunchConfig_t cfg{};
  cfg.gridDim = dim3(C);
  cfg.blockDim = dim3(nt < 32 ? 32 : nt);
  cfg.dynamicSmemBytes = 0;
  cfg.stream = s;
  cudaLaunchAttribute at[2];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = C;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  int na = 1;
  if (g_pdl) {
    at[1].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[1].val.programmaticStreamSerializationAllowed = 1;
    na = 2;
  }
  cfg.attrs = at;
  cfg.numAttrs = na;
  return cudaLaunchKernelEx(&cfg, k_reduce_cl<TWO>, partials, nrb, nt, lpt, op, st, out, due, partials2) ==
         cudaSuccess;
}
int launch_reduce(const double* partials, int64_t nrb, double* roots, uint32_t* ticket, int op, CgState* st,
                  double* out, const int* due, cudaStream_t s) {
  int64_t p2 = 1;
  while (p2 < nrb) p2 <<= 1;
  if (launch_reduce_cl<false>(partials, nullptr, nrb, p2, op, st, out, due, s)) return 1;
  int64_t leaves = p2 < 1024 ? p2 : 1024;
  int blocks = (int)(p2 / leaves);
  launch_k(k_reduce<false>, blocks, 256, 0, s, partials, nrb, leaves, roots, ticket, op, st, out, due,
           (const double*)nullptr, (double*)nullptr);
  return 1;
}
int launch_reduce_sr(const double* partials, const double* partials2, int64_t nrb, double* roots, double* roots2,
                     uint32_t* ticket, int op, CgState* st, const int* due, cudaStream_t s) {
  int64_t p2 = 1;
  while (p2 < nrb) p2 <<= 1;
  if (launch_reduce_cl<true>(partials, partials2, nrb, p2, op, st, nullptr, due, s)) return 1;
  int64_t leaves = p2 < 1024 ? p2 : 1024;
  int blocks = (int)(p2 / leaves);
  launch_k(k_reduce<true>, blocks, 256, 0, s, partials, nrb, leaves, roots, ticket, op, st, (double*)nullptr, due,
           partials2, roots2);
  return 1;
}

int launch_reduce_sr_root(const double* partials, const double* partials2, int64_t nrb, double* roots, double* roots2,
                          uint32_t* ticket, double* out, const int* due, cudaStream_t s) {
  int64_t p2 = 1;
  while (p2 < nrb) p2 <<= 1;
  int64_t leaves = p2 < 1024 ? p2 : 1024;
  int blocks = (int)(p2 / leaves);
  if (launch_reduce_cl<true>(partials, partials2, nrb, p2, 10, nullptr, out, due, s)) return 1;
  launch_k(k_reduce<true>, blocks, 256, 0, s, partials, nrb, leaves, roots, ticket, 10, (CgState*)nullptr, out, due,
           partials2, roots2);
  return 1;
}
int launch_combine_sr(const double* gathered, int P, int op, CgState* st, int* due, cudaStream_t s) {
  k_combine_sr<<<1, 512, 0, s>>>(gathered, P, op, st, due);
  return 1;
}
int launch_combine(const double* gathered, int P, int op, CgState* st, int* due, cudaStream_t s) {
  k_combine<<<1, 512, 0, s>>>(gathered, P, op, st, due);
  return 1;
}
int launch_due_combine(const double* gathered, int P, CgState* st, int* due, cudaStream_t s) {
  k_due_combine<<<1, 1, 0, s>>>(gathered, P, st, due);
  return 1;
}
int launch_pack_due(double* out, const int* due, cudaStream_t s) {
  k_pack_due<<<1, 1, 0, s>>>(out, due);
  return 1;
}

int launch_csr_encode(abft_csr* A, uint32_t* flags, cudaStream_t s) {
  int launches = 0;
  uint64_t* val = reinterpret_cast<uint64_t*>(A->val);
  const int es = A->elem_scheme, rs = A->rowptr_scheme;
  if (A->nnz > 0 && es != NONE && es != CRC32C) {
    int nb = grid_for(A->nnz, 256);
    if (es == SED) k_encode_elems<SED><<<nb, 256, 0, s>>>(val, A->col, A->nnz, A->ncols, flags);
    else k_encode_elems<SECDED64><<<nb, 256, 0, s>>>(val, A->col, A->nnz, A->ncols, flags);
    launches++;
  }
  if (es == CRC32C && A->nrows > 0) {
    k_encode_elems<CRC32C><<<grid_for(A->nnz, 256), 256, 0, s>>>(val, A->col, A->nnz, A->ncols, flags);
    k_encode_ecrc<<<grid_for(A->nrows, 256), 256, 0, s>>>(val, A->col, A->rowptr, A->nrows, flags);
    launches += 2;
  }
  const int64_t len = rowptr_padded_len(A->nrows, rs);
  const int nb = grid_for(len, 256);
  switch (rs) {
    case NONE: k_encode_rowptr<NONE><<<nb, 256, 0, s>>>(A->rowptr, A->nrows, A->nnz, len, flags); break;
    case SED: k_encode_rowptr<SED><<<nb, 256, 0, s>>>(A->rowptr, A->nrows, A->nnz, len, flags); break;
    case SECDED64: k_encode_rowptr<SECDED64><<<nb, 256, 0, s>>>(A->rowptr, A->nrows, A->nnz, len, flags); break;
    case SECDED128: k_encode_rowptr<SECDED128><<<nb, 256, 0, s>>>(A->rowptr, A->nrows, A->nnz, len, flags); break;
    default: k_encode_rowptr<CRC32C><<<nb, 256, 0, s>>>(A->rowptr, A->nrows, A->nnz, len, flags); break;
  }
  return launches + 1;
}

template <int ES>
static int check_rows_es(const abft_csr* A, DevCounts* c, int* due, int scrub, cudaStream_t s) {
  int nb = grid_for(A->nrows, 256);
  uint64_t* val = reinterpret_cast<uint64_t*>(A->val);
  switch (A->rowptr_scheme) {
    case NONE: k_check_rows<ES, NONE><<<nb, 256, 0, s>>>(val, A->col, A->rowptr, A->nrows, A->nnz, A->ncols, c, due, scrub); break;
    case SED: k_check_rows<ES, SED><<<nb, 256, 0, s>>>(val, A->col, A->rowptr, A->nrows, A->nnz, A->ncols, c, due, scrub); break;
    case SECDED64: k_check_rows<ES, SECDED64><<<nb, 256, 0, s>>>(val, A->col, A->rowptr, A->nrows, A->nnz, A->ncols, c, due, scrub); break;
    case SECDED128: k_check_rows<ES, SECDED128><<<nb, 256, 0, s>>>(val, A->col, A->rowptr, A->nrows, A->nnz, A->ncols, c, due, scrub); break;
    default: k_check_rows<ES, CRC32C><<<nb, 256, 0, s>>>(val, A->col, A->rowptr, A->nrows, A->nnz, A->ncols, c, due, scrub); break;
  }
  return 1;
}

int launch_check_csr(const abft_csr* A, DevCounts* c, int* due, int scrub, cudaStream_t s) {
  int launches = 0;
  uint64_t* val = reinterpret_cast<uint64_t*>(A->val);
  const int es = A->elem_scheme, rs = A->rowptr_scheme;
  if (A->nnz > 0 && (es == SED || es == SECDED64 || es == SECDED128)) {
    int nb = grid_for(A->nnz, 256);
    if (es == SED) k_check_elems<SED><<<nb, 256, 0, s>>>(val, A->col, A->nnz, A->ncols, c, due, scrub);
    else k_check_elems<SECDED64><<<nb, 256, 0, s>>>(val, A->col, A->nnz, A->ncols, c, due, scrub);
    launches++;
  }
  const int64_t len = rowptr_padded_len(A->nrows, rs);
  if (rs != NONE) {
    int nb = grid_for(len, 256);
    switch (rs) {
      case SED: k_check_rowptr<SED><<<nb, 256, 0, s>>>(A->rowptr, len, c, due, scrub); break;
      case SECDED64: k_check_rowptr<SECDED64><<<nb, 256, 0, s>>>(A->rowptr, len, c, due, scrub); break;
      case SECDED128: k_check_rowptr<SECDED128><<<nb, 256, 0, s>>>(A->rowptr, len, c, due, scrub); break;
      default: k_check_rowptr<CRC32C><<<nb, 256, 0, s>>>(A->rowptr, len, c, due, scrub); break;
    }
    launches++;
  }
  if (A->nrows > 0 && (rs != NONE || es == CRC32C)) {
    if (es == CRC32C) launches += check_rows_es<CRC32C>(A, c, due, scrub, s);
    else launches += check_rows_es<NONE>(A, c, due, scrub, s);
  }
  return launches;
}

static __global__ void k_inject_sched(const DevFault* f, int n, const CgState* st, int phase) {
  if (phase && st->stop) return;
  const int k = phase ? st->iters + 1 : 0;
  for (int i = threadIdx.x; i < n; i += blockDim.x)
    if (f[i].iter == k) atomicXor(f[i].addr, f[i].mask);
}
int launch_inject_sched(const DevFault* f, int n, const CgState* st, int phase, cudaStream_t s) {
  if (n <= 0) return 0;
  k_inject_sched<<<1, 256, 0, s>>>(f, n, st, phase);
  return 1;
}

int launch_wait_halo(const int* flags, const CgState* st, int need_up, int need_dn, cudaStream_t s) {
  k_wait_halo<<<1, 1, 0, s>>>(flags, st, need_up, need_dn);
  return 1;
}
int launch_inject(void* base, uint64_t bit, cudaStream_t s) {
  k_inject<<<1, 1, 0, s>>>(reinterpret_cast<uint32_t*>(base), bit);
  return 1;
}

int64_t rowptr_padded_len(int64_t nrows, int scheme) {
  int64_t g = rgrp(scheme);
  return (nrows + 1 + g - 1) / g * g;
}
int64_t vec_padded_len(int64_t n, int scheme) {
  int64_t g = vgrp(scheme);
  return (n + g - 1) / g * g;
}

}  // namespace abft

// Host hooks: run the exact codec functions on the CPU (unit tests vs oracle).
extern "C" int abft_codec_host_check(int inst, uint32_t* w) {
  using namespace abft;
  int word = 0;
  switch (inst) {
    case 0: {
      uint64_t v = mk64(w[0], w[1]);
      uint32_t c = w[2];
      int o = e96_bad(w[0], w[1], w[2]) ? e96_correct(v, c, &word) : CLEAN;
      if (o == CORRECTED) { w[0] = lo32(v); w[1] = hi32(v); w[2] = c; }
      return o;
    }
    case 1: {
      uint64_t u = mk64(w[0], w[1]);
      int o = vec_check_group<SECDED64>(&u, &word);
      if (o == CORRECTED) { w[0] = lo32(u); w[1] = hi32(u); }
      return o;
    }
    case 2: return rp_check_group<SECDED64>(w, &word);
    case 3: return rp_check_group<SECDED128>(w, &word);
    case 4: {
      uint64_t d[2] = {mk64(w[0], w[1]), mk64(w[2], w[3])};
      int o = v128_check(d, &word);
      if (o == CORRECTED) { w[0] = lo32(d[0]); w[1] = hi32(d[0]); w[2] = lo32(d[1]); w[3] = hi32(d[1]); }
      return o;
    }
    case 5: {   // the tiled SpMV's pair-packed E-SECDED fast check of two codewords w[0..2], w[3..5]
      uint32_t u = 0, p = 0;
      e96_acc2(w[0], w[1], w[2], w[3], w[4], w[5], u, p);
      return ((u & MOEB2_SYN_MASK) | (p & 1u)) ? DUE : CLEAN;
    }
    case 6: {   // the decoded window's pair-packed V-SECDED64 fast check of w[0..1], w[2..3]
      uint32_t u = 0, p = 0;
      v64_acc2(w[0], w[1], w[2], w[3], u, p);
      return ((u & MOEB2_SYN_MASK) | (p & 1u)) ? DUE : CLEAN;
    }
  }
  return -1;
}
extern "C" void abft_codec_host_encode(int inst, uint32_t* w) {
  using namespace abft;
  switch (inst) {
    case 0: w[2] = e96_encode_col(mk64(w[0], w[1]), w[2]); break;
    case 1: {
      uint64_t u = v64_encode_lut(mk64(w[0], w[1]) & ~0xFFull, h_v64_lut.r);
      w[0] = lo32(u); w[1] = hi32(u);
      break;
    }
    case 2: rp_encode_group<SECDED64>(w); break;
    case 3: rp_encode_group<SECDED128>(w); break;
    case 4: {
      uint64_t d[2] = {mk64(w[0], w[1]) & ~0x1Full, mk64(w[2], w[3]) & ~0x1Full};
      v128_encode(d);
      w[0] = lo32(d[0]); w[1] = hi32(d[0]); w[2] = lo32(d[1]); w[3] = hi32(d[1]);
      break;
    }
  }
}
