// capi.cu — the C ABI of libabft.so (include/abft.h): argument validation,
// scratch ownership, and the device-resident CG driver.
// Host code only; every arithmetic step runs in kernels.cu.
#include <cuda.h>
#include <cudaTypedefs.h>
#include <cuda_runtime.h>

#include <atomic>
#include <cstdarg>
#include <cmath>
#include <cstdio>
#include <cstring>
#include <string>
#include <vector>

#include <nccl.h>

#include "../../include/abft.h"
#include "internal.h"

using namespace abft;

static thread_local std::string g_err;
static std::atomic<uint64_t> g_launches{0};

static int fail(int code, const char* fmt, ...) __attribute__((format(printf, 2, 3)));
static int fail(int code, const char* fmt, ...) {
  char buf[512];
  va_list ap;
  va_start(ap, fmt);
  vsnprintf(buf, sizeof buf, fmt, ap);
  va_end(ap);
  g_err = buf;
  return code;
}
#define CUDA_TRY(x)                                                                          \
  do {                                                                                       \
    cudaError_t e_ = (x);                                                                    \
    if (e_ != cudaSuccess) return fail(ABFT_E_CUDA, "%s: %s", #x, cudaGetErrorString(e_)); \
  } while (0)

static inline void count_launch(int n) { g_launches.fetch_add((uint64_t)n, std::memory_order_relaxed); }

struct abft_ctx {
  int device = 0;
  double* partials = nullptr;
  double* partials2 = nullptr;  // second dot of the single-reduction CG's SpMV (same capacity)
  int64_t partials_cap = 0;
  double* roots2 = nullptr;
  double* roots = nullptr;
  uint32_t* ticket = nullptr;
  CgState* state = nullptr;
  int* due = nullptr;
  uint32_t* flags = nullptr;
  CgState* h_state = nullptr;  // pinned
  uint32_t* h_flags = nullptr; // pinned
  int profile = 0;        // bitmask of kernel classes to time: 1 SpMV, 2 calc_ur, 4 calc_p, 8 reductions
  bool use_graphs = true; // capture poll_every iterations into a CUDA graph (single GPU)
  cudaStream_t cap_stream = nullptr;
  double prof_ms[4] = {0, 0, 0, 0};
  int64_t prof_n[4] = {0, 0, 0, 0};
  std::vector<cudaEvent_t> events;
  CrcTables* crc = nullptr;  // CRC32C lookup tables (device)
  bool fuse_p = false;       // fused calc_p in the CG's SpMV when eligible (opt-in)
  bool pdl = false;          // programmatic dependent launch between the CG iteration kernels (opt-in, §6.2)
  uint64_t* p_alt = nullptr; // second p buffer of the fused CG
  int64_t p_alt_len = 0;
  double* cg_log = nullptr;   // [2 * CG_LOG]: CG alpha / beta of the first iterations (abft_cg_spectrum)
  DevFault* faults = nullptr; // O10 fault schedule applied by the next CG solves (abft_ctx_set_faults)
  int nfaults = 0;
};

namespace {

int ensure_partials(abft_ctx* c, int64_t nrb) {
  if (nrb <= c->partials_cap) return ABFT_OK;
  if (c->partials) cudaFree(c->partials);
  if (c->partials2) cudaFree(c->partials2);
  c->partials = c->partials2 = nullptr;
  c->partials_cap = 0;
  int64_t cap = nrb < 1024 ? 1024 : nrb;
  CUDA_TRY(cudaMalloc(&c->partials, sizeof(double) * cap));
  CUDA_TRY(cudaMalloc(&c->partials2, sizeof(double) * cap));
  c->partials_cap = cap;
  return ABFT_OK;
}

bool valid_scheme(int s) { return s >= 0 && s < ABFT_SCHEME_COUNT; }

int check_vec(const abft_vec* v, const char* name) {
  if (!v || !v->data || v->n < 0 || !valid_scheme(v->scheme)) return fail(ABFT_E_INVALID, "bad vector %s", name);
  return ABFT_OK;
}

int check_chunks(const abft_csr* A, int nchunks) {
  if (!A || nchunks <= 0) return fail(ABFT_E_INVALID, "no matrix chunks");
  for (int c = 0; c < nchunks; c++) {
    const abft_csr& M = A[c];
    if (M.nrows < 0 || M.ncols < 0 || M.nnz < 0 || !M.rowptr || (M.nnz > 0 && (!M.val || !M.col)))
      return fail(ABFT_E_INVALID, "chunk %d: bad sizes/pointers", c);
    if (!valid_scheme(M.elem_scheme) || !valid_scheme(M.rowptr_scheme))
      return fail(ABFT_E_INVALID, "chunk %d: bad scheme", c);
    if (M.row_base < 0 || M.col_base < 0) return fail(ABFT_E_INVALID, "chunk %d: negative base", c);
  }
  return ABFT_OK;
}

// Launch the SpMV over all chunks; partials indexed by global RB (chunks must
// start on 256-row boundaries relative to chunk 0 when dot is requested).
// fused calc_p (CG driver): p_cur != null => in = p_{k-1}, r_f = r;
// probe = true only builds the arguments and reports whether every chunk can
// take the fused tiled kernel (nothing is launched).
int spmv_chunks(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* in, abft_vec* out, int dot,
                DevCounts* cnt, const CgState* st, cudaStream_t s, int64_t* nrb_total,
                int check_mode = MODE_CORRECT, int check_interval = 0, uint64_t* p_cur = nullptr,
                uint64_t* r_f = nullptr, bool probe = false, int part = 0, bool early_in = false) {
  const int64_t base0 = A[0].row_base;
  const int64_t npad_in = vec_padded_len(in->n, in->scheme);
  const int64_t npad_out = vec_padded_len(out->n, out->scheme);
  int64_t nrb_all = 0;
  for (int c = 0; c < nchunks; c++) {
    const abft_csr& M = A[c];
    const int64_t rel = M.row_base - base0;
    if (dot && (rel % 256) != 0) return fail(ABFT_E_INVALID, "chunk %d not aligned to 256 rows", c);
    const int64_t end_rb = (rel + M.nrows + 255) / 256;
    if (end_rb > nrb_all) nrb_all = end_rb;
  }
  if (dot && !probe) {
    int e = ensure_partials(ctx, nrb_all);
    if (e) return e;
  }
  for (int c = 0; c < nchunks; c++) {
    const abft_csr& M = A[c];
    if (M.row_base + M.nrows > out->n) return fail(ABFT_E_INVALID, "chunk %d rows exceed out", c);
    // lane groups of G > 1 vector codecs (V-SECDED128 pairs, V-CRC quads) must
    // line up with the stored codeword groups
    if (M.row_base % vec_padded_len(1, out->scheme) != 0)
      return fail(ABFT_E_SHAPE, "chunk %d: row_base not a multiple of the vector group size", c);
    if (M.col_base + M.ncols > npad_in) return fail(ABFT_E_INVALID, "chunk %d cols exceed in", c);
    SpmvArgs a{};
    a.nrows = M.nrows;
    a.ncols = M.ncols;
    a.nnz = M.nnz;
    a.row_base = M.row_base;
    a.col_base = M.col_base;
    a.n_in = in->n;
    a.npad_in = npad_in;
    a.npad_out = (M.row_base + M.nrows == out->n) ? (npad_out - M.row_base) : M.nrows;
    a.rb_offset = (M.row_base - base0) / 256;
    a.stencil_n = M.stencil_n;
    a.val = reinterpret_cast<uint64_t*>(M.val);
    a.col = M.col;
    a.rowptr = M.rowptr;
    a.in = reinterpret_cast<uint64_t*>(in->data);
    a.out = reinterpret_cast<uint64_t*>(out->data);
    a.partials = dot ? ctx->partials : nullptr;
    a.partials2 = dot == 2 ? ctx->partials2 : nullptr;
    a.counts = cnt;
    a.due = ctx->due;
    a.state = st;
    a.check_mode = check_mode;
    a.check_interval = check_interval;
    a.crc = ctx->crc;
    a.p_cur = p_cur;
    a.r_f = r_f;
    a.early_in = early_in ? 1 : 0;
    if (probe) {
      // probe: p_cur set -> can the fused calc_p kernel run; else -> is every chunk tileable
      if (p_cur ? !spmv_fusable(a, in->scheme) : !spmv_tileable(a, in->scheme)) return ABFT_E_SHAPE;
      continue;
    }
    if (part != 0) {
      // halo overlap (multi-rank, every chunk tileable): part 1 = the interior
      // tile rows, whose windows never reach the ghost rows; part 2 = the first
      // tile row of the first chunk and the last of the last chunk
      const int64_t nty = spmv_tile_rows(a);
      const int64_t lo = (c == 0) ? 1 : 0;
      int64_t hi = (c == nchunks - 1) ? nty - 1 : nty;
      if (hi < lo) hi = lo;
      int64_t rng[2][2] = {{lo, hi}, {0, 0}};
      if (part == 2) { rng[0][0] = 0; rng[0][1] = lo; rng[1][0] = hi; rng[1][1] = nty; }
      for (int q = 0; q < 2; q++) {
        if (rng[q][1] <= rng[q][0]) continue;
        a.ty_lo = rng[q][0];
        a.ty_hi = rng[q][1];
        const int l = launch_spmv(a, M.elem_scheme, M.rowptr_scheme, in->scheme, dot, s);
        if (l < 0) return fail(ABFT_E_CUDA, "chunk %d: SpMV part could not be launched", c);
        count_launch(l);
      }
      continue;
    }
    const int l = launch_spmv(a, M.elem_scheme, M.rowptr_scheme, in->scheme, dot, s);
    if (l < 0) return fail(ABFT_E_CUDA, "chunk %d: fused calc_p SpMV could not be launched", c);
    count_launch(l);
  }
  if (nrb_total) *nrb_total = nrb_all;
  return ABFT_OK;
}

}  // namespace

extern "C" {

const char* abft_last_error(void) { return g_err.c_str(); }
uint64_t abft_launch_count(void) { return g_launches.load(); }

int64_t abft_rowptr_padded_len(int64_t nrows, int32_t scheme) { return rowptr_padded_len(nrows, scheme); }
int64_t abft_vec_padded_len(int64_t n, int32_t scheme) { return vec_padded_len(n, scheme); }

int abft_ctx_create(int device, abft_ctx** out) {
  if (!out) return fail(ABFT_E_INVALID, "null out");
  CUDA_TRY(cudaSetDevice(device));
  abft_ctx* c = new abft_ctx();
  c->device = device;
  CUDA_TRY(cudaMalloc(&c->roots, sizeof(double) * 1024));
  CUDA_TRY(cudaMalloc(&c->roots2, sizeof(double) * 1024));
  CUDA_TRY(cudaMalloc(&c->cg_log, sizeof(double) * 2 * CG_LOG));
  CUDA_TRY(cudaMalloc(&c->ticket, sizeof(uint32_t) * 4));
  CUDA_TRY(cudaMemset(c->ticket, 0, sizeof(uint32_t) * 4));
  CUDA_TRY(cudaMalloc(&c->state, sizeof(CgState)));
  CUDA_TRY(cudaMemset(c->state, 0, sizeof(CgState)));
  CUDA_TRY(cudaMalloc(&c->due, sizeof(int) * 4));
  CUDA_TRY(cudaMemset(c->due, 0, sizeof(int) * 4));
  CUDA_TRY(cudaMalloc(&c->flags, sizeof(uint32_t) * 4));
  CUDA_TRY(cudaMallocHost(&c->h_state, sizeof(CgState)));
  CUDA_TRY(cudaMallocHost(&c->h_flags, sizeof(uint32_t) * 4));
  {
    std::vector<CrcTables> h(1);
    build_crc_tables(h.data());
    CUDA_TRY(cudaMalloc(&c->crc, sizeof(CrcTables)));
    CUDA_TRY(cudaMemcpy(c->crc, h.data(), sizeof(CrcTables), cudaMemcpyHostToDevice));
  }
  prepare_kernels(device);
  int e = ensure_partials(c, 1024);
  if (e) return e;
  *out = c;
  return ABFT_OK;
}

int abft_ctx_set_pdl(abft_ctx* c, int enable) {
  if (!c) return fail(ABFT_E_INVALID, "null ctx");
  c->pdl = enable != 0;
  return ABFT_OK;
}

int abft_ctx_set_crc_correction(abft_ctx* c, int bits) {
  if (!c || (bits != 1 && bits != 2)) return fail(ABFT_E_INVALID, "CRC32C correction: 1 (1EC4ED) or 2 (2EC3ED)");
  CUDA_TRY(cudaSetDevice(c->device));
  CUDA_TRY(cudaMemcpy(c->due + 1, &bits, sizeof(int), cudaMemcpyHostToDevice));   // cfg[1] (crc_t_of)
  return ABFT_OK;
}

int abft_ctx_set_fused_cg(abft_ctx* c, int enable) {
  if (!c) return fail(ABFT_E_INVALID, "null ctx");
  c->fuse_p = enable != 0;
  return ABFT_OK;
}

int abft_ctx_destroy(abft_ctx* c) {
  if (!c) return ABFT_OK;
  cudaSetDevice(c->device);
  cudaFree(c->partials);
  cudaFree(c->partials2);
  cudaFree(c->roots);
  cudaFree(c->roots2);
  cudaFree(c->ticket);
  cudaFree(c->state);
  cudaFree(c->due);
  cudaFree(c->flags);
  cudaFree(c->p_alt);
  cudaFree(c->faults);
  cudaFree(c->cg_log);
  cudaFree(c->crc);
  cudaFreeHost(c->h_state);
  cudaFreeHost(c->h_flags);
  for (auto e : c->events) cudaEventDestroy(e);
  if (c->cap_stream) cudaStreamDestroy(c->cap_stream);
  delete c;
  return ABFT_OK;
}

int abft_csr_encode(abft_ctx* ctx, abft_csr* A, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  int e = check_chunks(A, 1);
  if (e) return e;
  cudaStream_t s = (cudaStream_t)stream;
  const uint64_t cap_col = A->elem_scheme == ABFT_NONE ? 0xFFFFFFFFull
                           : A->elem_scheme == ABFT_SED ? 0x7FFFFFFFull : 0x00FFFFFFull;
  const uint64_t cap_nnz = A->rowptr_scheme == ABFT_NONE ? 0xFFFFFFFFull
                           : A->rowptr_scheme == ABFT_SED ? 0x7FFFFFFFull : 0x0FFFFFFFull;
  if (A->ncols > 0 && (uint64_t)(A->ncols - 1) > cap_col)
    return fail(ABFT_E_RANGE, "ncols %lld exceeds the element scheme's index capacity", (long long)A->ncols);
  if ((uint64_t)A->nnz > cap_nnz) return fail(ABFT_E_RANGE, "nnz %lld exceeds the rowptr scheme's capacity", (long long)A->nnz);
  CUDA_TRY(cudaMemsetAsync(ctx->flags, 0, sizeof(uint32_t), s));
  count_launch(launch_csr_encode(A, ctx->flags, s));
  CUDA_TRY(cudaGetLastError());
  CUDA_TRY(cudaMemcpyAsync(ctx->h_flags, ctx->flags, sizeof(uint32_t), cudaMemcpyDeviceToHost, s));
  CUDA_TRY(cudaStreamSynchronize(s));
  uint32_t f = ctx->h_flags[0];
  if (f & 4u) return fail(ABFT_E_SHAPE, "CRC32C element rows need >= 4 entries");
  if (f & 3u) return fail(ABFT_E_RANGE, "column index or rowptr entry exceeds the scheme's capacity");
  return ABFT_OK;
}

int abft_vec_encode(abft_ctx* ctx, abft_vec* v, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  int e = check_vec(v, "v");
  if (e) return e;
  count_launch(launch_vec_encode(reinterpret_cast<uint64_t*>(v->data), v->n, vec_padded_len(v->n, v->scheme),
                                 v->scheme, (cudaStream_t)stream));
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

int abft_vec_decode(abft_ctx* ctx, abft_vec* v, double* out_masked, abft_counts* dcnt, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  int e = check_vec(v, "v");
  if (e) return e;
  count_launch(launch_vec_check(reinterpret_cast<uint64_t*>(v->data), v->n, vec_padded_len(v->n, v->scheme),
                                v->scheme, out_masked, reinterpret_cast<DevCounts*>(dcnt), ctx->due, 1,
                                (cudaStream_t)stream));
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

int abft_spmv(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* in, abft_vec* out, double* dot_out,
              abft_counts* dcnt, void* stream) {
  return abft_spmv_ex(ctx, A, nchunks, in, out, dot_out, dcnt, ABFT_CHECK_CORRECT, stream);
}

int abft_spmv_ex(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* in, abft_vec* out, double* dot_out,
                 abft_counts* dcnt, int32_t check_mode, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  if (check_mode < ABFT_CHECK_CORRECT || check_mode > ABFT_CHECK_RANGE) return fail(ABFT_E_INVALID, "bad check mode");
  int e = check_chunks(A, nchunks);
  if (e) return e;
  if ((e = check_vec(in, "in")) || (e = check_vec(out, "out"))) return e;
  if (in->data == out->data) return fail(ABFT_E_INVALID, "in and out alias");
  if (in->scheme != out->scheme) return fail(ABFT_E_INVALID, "in/out schemes differ");
  cudaStream_t s = (cudaStream_t)stream;
  int64_t nrb = 0;
  e = spmv_chunks(ctx, A, nchunks, in, out, dot_out != nullptr, reinterpret_cast<DevCounts*>(dcnt), nullptr, s, &nrb,
                  check_mode);
  if (e) return e;
  if (dot_out) count_launch(launch_reduce(ctx->partials, nrb, ctx->roots, ctx->ticket, 0, nullptr, dot_out, ctx->due, s));
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

int abft_spmv_partials(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* in, abft_vec* out, abft_counts* dcnt,
                       void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  int e = check_chunks(A, nchunks);
  if (e) return e;
  if ((e = check_vec(in, "in")) || (e = check_vec(out, "out"))) return e;
  if (in->data == out->data) return fail(ABFT_E_INVALID, "in and out alias");
  if (in->scheme != out->scheme) return fail(ABFT_E_INVALID, "in/out schemes differ");
  cudaStream_t s = (cudaStream_t)stream;
  int64_t nrb = 0;
  e = spmv_chunks(ctx, A, nchunks, in, out, true, reinterpret_cast<DevCounts*>(dcnt), nullptr, s, &nrb,
                  ABFT_CHECK_CORRECT);
  if (e) return e;
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

int abft_profile(abft_ctx* ctx, int enable) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  ctx->profile = enable;
  for (int i = 0; i < 4; i++) { ctx->prof_ms[i] = 0; ctx->prof_n[i] = 0; }
  return ABFT_OK;
}
int abft_profile_read(abft_ctx* ctx, double* ms, int64_t* n) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  for (int i = 0; i < 4; i++) { if (ms) ms[i] = ctx->prof_ms[i]; if (n) n[i] = ctx->prof_n[i]; }
  return ABFT_OK;
}

// --------------------------------------------------------------------- CG
namespace {

struct Prof {
  abft_ctx* ctx;
  cudaStream_t s;
  std::vector<std::pair<int, int>> marks;  // (class, event index of start)
  size_t next = 0;
  cudaEvent_t ev(size_t i) {
    while (ctx->events.size() <= i) {
      cudaEvent_t e;
      cudaEventCreate(&e);
      ctx->events.push_back(e);
    }
    return ctx->events[i];
  }
  bool on = false;
  void begin(int cls) {
    on = (ctx->profile >> cls) & 1;
    if (!on) return;
    cudaEventRecord(ev(next), s);
    marks.push_back({cls, (int)next});
    next += 2;
  }
  void end() {
    if (!on) return;
    cudaEventRecord(ev(marks.back().second + 1), s);
    on = false;
  }
  void harvest(bool keep = false) {  // after a stream sync; keep = marks belong to a graph
    if (!ctx->profile) return;
    for (auto& m : marks) {
      float ms = 0;
      if (cudaEventElapsedTime(&ms, ctx->events[m.second], ctx->events[m.second + 1]) == cudaSuccess) {
        ctx->prof_ms[m.first] += ms;
        ctx->prof_n[m.first] += 1;
      } else {
        (void)cudaGetLastError();  // a failed timing query must not poison later calls
      }
    }
    if (!keep) {
      marks.clear();
      next = 0;
    }
  }
};

}  // namespace

}  // extern "C"

// ------------------------------------------------------------ multi-rank plumbing
// abft_dist is the transport of the row-block strips: NCCL with
// one rank per process in production, or an in-process LOOPBACK of P virtual
// ranks on one device (every rank's vectors in this process) that runs the same
// per-rank kernel sequence, halo and all-gather points for testing the P > 1
// path without a second GPU.  Both expose the two exchange steps the CG
// iteration has: the p halo (one grid row each side) and the all-gather of one
// (RED-1 subtree root, DUE flag) pair per rank.
struct abft_dist {
  int loopback = 0;
  ncclComm_t comm = nullptr;
  int rank = 0, nranks = 1, device = 0;
  double* sendbuf = nullptr;   // NCCL: this rank's pair [2]
  double* gathered = nullptr;  // all ranks' payloads [GATHER_W * nranks] (loopback: rank r writes its own slot)
  cudaStream_t comm_stream = nullptr;   // halo exchange, overlapped with the interior SpMV
  cudaEvent_t ev_fork = nullptr, ev_join = nullptr;
  // peer-memory halos (S§8(f) f3): p's ghost rows are stored by
  // the neighbours' calc_p straight into this rank's vector; arrival flags
  int peer_halo = 0;
  int* flags = nullptr;         // [2] this rank's (NCCL) / [2 * nranks] every loopback rank's: [0] from rank-1, [1] from rank+1
  uint64_t* peer_p[2] = {};     // NCCL: the neighbours' halo-extended p, mapped here ([0] rank-1, [1] rank+1)
  int* peer_flag[2] = {};       // NCCL: where this rank signals: rank-1's flags[1], rank+1's flags[0] (mapped)
};

namespace {

#define NCCL_TRY(x)                                                                        \
  do {                                                                                     \
    ncclResult_t r_ = (x);                                                                 \
    if (r_ != ncclSuccess) return fail(ABFT_E_NCCL, "%s: %s", #x, ncclGetErrorString(r_)); \
  } while (0)

// One rank's share of a (possibly distributed) CG solve.
struct RankRun {
  abft_ctx* ctx = nullptr;
  const abft_csr* A = nullptr;
  int nchunks = 0;
  abft_vec* v[5] = {};   // b x r p w
  abft_vec* s_vec = nullptr;   // single-reduction CG: its extra vector s
  VecArgs va_sr{};
  bool cheb = false;           // Chebyshev iteration with bounds [eigmin, eigmax]; x is u
  double eigmin = 0.0, eigmax = 0.0;
  int ppcg_inner = 0;          // PPCG: inner Chebyshev steps; z, rin, pin its vectors
  abft_vec* z = nullptr;
  abft_vec* rin = nullptr;
  abft_vec* pin = nullptr;
  DevCounts* cnt = nullptr;
  int64_t n = 0, nrb = 0, n_ext = 0;
  VecArgs va{};
  double* sendbuf = nullptr;
  double* gathered = nullptr;
  abft_vec* b() const { return v[0]; }
  abft_vec* x() const { return v[1]; }
  abft_vec* r() const { return v[2]; }
  abft_vec* p() const { return v[3]; }
  abft_vec* w() const { return v[4]; }
};

int validate_rank(RankRun& R, int64_t n_halo, const abft_cg_opts* opts) {
  int e = check_chunks(R.A, R.nchunks);
  if (e) return e;
  const char* names[5] = {"b", "x", "r", "p", "w"};
  for (int i = 0; i < 5; i++) if ((e = check_vec(R.v[i], names[i]))) return e;
  const int scheme = R.x()->scheme;
  R.n_ext = R.x()->n;
  for (int i = 0; i < 5; i++) {
    if (R.v[i]->scheme != scheme || R.v[i]->n != R.n_ext) return fail(ABFT_E_INVALID, "vector %s: scheme/length differ", names[i]);
    for (int j = 0; j < i; j++) if (R.v[i]->data == R.v[j]->data) return fail(ABFT_E_INVALID, "vectors alias");
  }
  R.n = R.n_ext - 2 * n_halo;  // local rows
  const int G = (int)vec_padded_len(1, scheme);
  if (R.n <= 0 || n_halo < 0 || (n_halo % G) != 0) return fail(ABFT_E_SHAPE, "bad halo / local size");
  if (n_halo > 0 && (R.n % G) != 0) return fail(ABFT_E_SHAPE, "local rows must be a multiple of the vector group");
  int64_t rows = 0;
  for (int c = 0; c < R.nchunks; c++) rows += R.A[c].nrows;
  if (R.A[0].row_base != n_halo || rows != R.n) return fail(ABFT_E_SHAPE, "chunks must cover the local rows");
  R.nrb = (R.n + 255) / 256;
  if ((e = ensure_partials(R.ctx, R.nrb))) return e;
  if (opts->check_interval < 0) return fail(ABFT_E_INVALID, "negative check interval");
  if (R.nrb > (int64_t)1024 * 1024) return fail(ABFT_E_SHAPE, "more than 2^28 rows per GPU");
  VecArgs& va = R.va;
  va = VecArgs{};
  va.n = R.n;
  va.npad = vec_padded_len(R.n, scheme);
  va.x = reinterpret_cast<uint64_t*>(R.x()->data) + n_halo;
  va.p = reinterpret_cast<uint64_t*>(R.p()->data) + n_halo;
  va.r = reinterpret_cast<uint64_t*>(R.r()->data) + n_halo;
  va.w = reinterpret_cast<uint64_t*>(R.w()->data) + n_halo;
  va.b = reinterpret_cast<uint64_t*>(R.b()->data) + n_halo;
  va.partials = R.ctx->partials;
  va.counts = R.cnt;
  va.due = R.ctx->due;
  va.state = R.ctx->state;
  va.crc = R.ctx->crc;
  return ABFT_OK;
}

// Exchange the ghost rows of vector `vi` (extended by n_halo entries each side)
// of every local rank with its strip neighbours, on stream s.
int halo_exchange(abft_dist* d, RankRun* R, int nl, int vi, int64_t n_halo, cudaStream_t s) {
  if (!d || d->nranks == 1 || n_halo == 0) return ABFT_OK;
  const size_t bytes = sizeof(uint64_t) * (size_t)n_halo;
  if (d->loopback) {
    // rank r's top ghost <- rank r-1's last local grid row; bottom ghost <- rank r+1's first
    for (int q = 0; q < nl; q++) {
      uint64_t* ext = reinterpret_cast<uint64_t*>(R[q].v[vi]->data);
      if (q > 0) {
        const uint64_t* up = reinterpret_cast<const uint64_t*>(R[q - 1].v[vi]->data);
        CUDA_TRY(cudaMemcpyAsync(ext, up + R[q - 1].n, bytes, cudaMemcpyDeviceToDevice, s));
      }
      if (q < nl - 1) {
        const uint64_t* dn = reinterpret_cast<const uint64_t*>(R[q + 1].v[vi]->data);
        CUDA_TRY(cudaMemcpyAsync(ext + n_halo + R[q].n, dn + n_halo, bytes, cudaMemcpyDeviceToDevice, s));
      }
    }
    return ABFT_OK;
  }
  uint64_t* ext = reinterpret_cast<uint64_t*>(R[0].v[vi]->data);
  const int64_t n_loc = R[0].n;
  NCCL_TRY(ncclGroupStart());
  if (d->rank > 0) {
    NCCL_TRY(ncclSend(ext + n_halo, bytes, ncclChar, d->rank - 1, d->comm, s));
    NCCL_TRY(ncclRecv(ext, bytes, ncclChar, d->rank - 1, d->comm, s));
  }
  if (d->rank < d->nranks - 1) {
    NCCL_TRY(ncclSend(ext + n_loc, bytes, ncclChar, d->rank + 1, d->comm, s));
    NCCL_TRY(ncclRecv(ext + n_halo + n_loc, bytes, ncclChar, d->rank + 1, d->comm, s));
  }
  NCCL_TRY(ncclGroupEnd());
  return ABFT_OK;
}

// every rank's (root, due) pair -> every rank's `gathered`
int allgather_pairs(abft_dist* d, cudaStream_t s) {
  if (d->loopback) return ABFT_OK;   // the ranks wrote their pairs into the one shared buffer
  NCCL_TRY(ncclAllGather(d->sendbuf, d->gathered, GATHER_W, ncclDouble, d->comm, s));
  return ABFT_OK;
}

// Dot-product finish: single GPU -> k_reduce applies `op`;
// multi-rank -> each rank's subtree root + DUE flag, all-gather, and the same
// top-of-tree combine on every rank (bit-identical to one GPU for aligned
// power-of-two subtrees).
int finish_dot(RankRun* R, int nl, abft_dist* d, int op, cudaStream_t s) {
  if (!d) {
    abft_ctx* c = R[0].ctx;
    count_launch(launch_reduce(c->partials, R[0].nrb, c->roots, c->ticket, op, c->state, nullptr, c->due, s));
    return ABFT_OK;
  }
  for (int q = 0; q < nl; q++) {
    abft_ctx* c = R[q].ctx;
    count_launch(launch_reduce(c->partials, R[q].nrb, c->roots, c->ticket, 4, nullptr, R[q].sendbuf, c->due, s));
  }
  int e = allgather_pairs(d, s);
  if (e) return e;
  for (int q = 0; q < nl; q++)
    count_launch(launch_combine(R[q].gathered, d->nranks, op, R[q].ctx->state, R[q].ctx->due, s));
  return ABFT_OK;
}

// Single-reduction CG's one reduction: both RED-1 trees;
// multi-rank -> (w.r root, DUE flag, r.r root) all-gathered, both tops of the
// tree combined identically on every rank.
int finish_sr(RankRun* R, int nl, abft_dist* d, int op, cudaStream_t s) {
  if (!d) {
    abft_ctx* c = R[0].ctx;
    count_launch(launch_reduce_sr(c->partials, c->partials2, R[0].nrb, c->roots, c->roots2, c->ticket, op, c->state,
                                  c->due, s));
    return ABFT_OK;
  }
  for (int q = 0; q < nl; q++) {
    abft_ctx* c = R[q].ctx;
    count_launch(launch_reduce_sr_root(c->partials, c->partials2, R[q].nrb, c->roots, c->roots2, c->ticket,
                                       R[q].sendbuf, c->due, s));
  }
  int e = allgather_pairs(d, s);
  if (e) return e;
  for (int q = 0; q < nl; q++)
    count_launch(launch_combine_sr(R[q].gathered, d->nranks, op, R[q].ctx->state, R[q].ctx->due, s));
  return ABFT_OK;
}

// The CG driver for nl local ranks in lockstep (nl = 1: one GPU, or one NCCL
// rank of a multi-process solve; nl = P: the loopback).  Every kernel runs on
// stream s; all CG scalars live on the device.
int cg_run(RankRun* R, int nl, abft_dist* d, int64_t n_halo, const abft_cg_opts* opts, abft_cg_result* res,
           cudaStream_t s) {
  if (!opts || !res) return fail(ABFT_E_INVALID, "null opts/res");
  for (int q = 0; q < nl; q++) {
    if (!R[q].ctx) return fail(ABFT_E_INVALID, "null ctx");
    int e = validate_rank(R[q], n_halo, opts);
    if (e) return e;
    for (int j = 0; j < q; j++)
      if (R[q].ctx == R[j].ctx) return fail(ABFT_E_INVALID, "loopback ranks need one context each");
  }
  abft_ctx* ctx = R[0].ctx;   // graphs, events, polling
  const int scheme = R[0].x()->scheme;
  // single-reduction CG (Chronopoulos-Gear, S§8(f) f3): one GPU, every access checked
  const bool sr = R[0].s_vec != nullptr;
  const bool cheb = R[0].cheb;
  const bool ppcg = R[0].ppcg_inner > 0;
  std::vector<double> pc_alpha, pc_beta;   // PPCG inner step coefficients (host, rounded as written)
  double pc_theta = 0.0;
  VecArgs vpc{}, vdot{}, vcp{};
  if (ppcg) {
    if (d || nl != 1) return fail(ABFT_E_SHAPE, "PPCG runs on one GPU");
    if (opts->check_interval > 1) return fail(ABFT_E_SHAPE, "PPCG checks every access");
    if (!(R[0].eigmax > R[0].eigmin)) return fail(ABFT_E_INVALID, "PPCG bounds need eigmax > eigmin");
    abft_vec* extra[3] = {R[0].z, R[0].rin, R[0].pin};
    for (int i = 0; i < 3; i++) {
      int e0 = check_vec(extra[i], "z/rin/pin");
      if (e0) return e0;
      if (extra[i]->scheme != scheme || extra[i]->n != R[0].n_ext)
        return fail(ABFT_E_INVALID, "PPCG vectors: scheme/length differ");
      for (int j = 0; j < 5; j++) if (R[0].v[j]->data == extra[i]->data) return fail(ABFT_E_INVALID, "vectors alias");
      for (int j = 0; j < i; j++) if (extra[j]->data == extra[i]->data) return fail(ABFT_E_INVALID, "vectors alias");
    }
    pc_theta = (R[0].eigmax + R[0].eigmin) / 2.0;
    const double delta = (R[0].eigmax - R[0].eigmin) / 2.0, sigma = pc_theta / delta;
    double rho = 1.0 / sigma;
    for (int j = 1; j < R[0].ppcg_inner; j++) {
      const double rho_new = 1.0 / (2.0 * sigma - rho);
      pc_alpha.push_back(rho_new * rho);
      pc_beta.push_back((2.0 * rho_new) / delta);
      rho = rho_new;
    }
    auto ptr = [](abft_vec* v) { return reinterpret_cast<uint64_t*>(v->data); };
    vpc = R[0].va;      // preconditioner: rhs r, u = z, direction pin, residual rin, A z -> w
    vpc.b = ptr(R[0].r());
    vpc.x = ptr(R[0].z);
    vpc.p = ptr(R[0].pin);
    vpc.r = ptr(R[0].rin);
    vdot = R[0].va;     // r . z
    vdot.x = ptr(R[0].z);
    vcp = R[0].va;      // p = z + beta p
    vcp.r = ptr(R[0].z);
  }
  if (cheb) {
    if (d || nl != 1) return fail(ABFT_E_SHAPE, "Chebyshev iteration runs on one GPU");
    if (opts->check_interval > 1) return fail(ABFT_E_SHAPE, "Chebyshev iteration checks every access");
    if (!(R[0].eigmax > R[0].eigmin)) return fail(ABFT_E_INVALID, "Chebyshev bounds need eigmax > eigmin");
  }
  if (sr) {
    if (opts->check_interval > 1) return fail(ABFT_E_SHAPE, "single-reduction CG checks every access");
    for (int q = 0; q < nl; q++) {
      if (!R[q].s_vec) return fail(ABFT_E_INVALID, "rank %d: null vector s", q);
      int e0 = check_vec(R[q].s_vec, "s");
      if (e0) return e0;
      if (R[q].s_vec->scheme != scheme || R[q].s_vec->n != R[q].n_ext)
        return fail(ABFT_E_INVALID, "vector s: scheme/length differ");
      for (int j = 0; j < 5; j++)
        if (R[q].v[j]->data == R[q].s_vec->data) return fail(ABFT_E_INVALID, "vectors alias");
      R[q].va_sr = R[q].va;   // the update's VecArgs.b carries s
      R[q].va_sr.b = reinterpret_cast<uint64_t*>(R[q].s_vec->data) + n_halo;
    }
  }
  const int G = (int)vec_padded_len(1, scheme);
  const int interval = opts->check_interval > 1 ? opts->check_interval : 0;
  // the dist path runs whenever a transport is given (also with 1 rank, so the
  // all-gather / top-of-tree combine code is exercised on a single GPU)
  const bool multi = d != nullptr;
  if (multi) {
    for (int q = 0; q < nl; q++) {
      R[q].sendbuf = d->loopback ? d->gathered + GATHER_W * q : d->sendbuf;
      R[q].gathered = d->gathered;
    }
  }
  int e;
  // fused calc_p: single GPU, every chunk on the tiled path,
  // G = 1 vector scheme; p is double-buffered with ctx->p_alt
  const int64_t npad_ext = vec_padded_len(R[0].n_ext, scheme);
  // (a fault schedule addresses the caller's p: the double-buffered fused CG is off then)
  bool fused = ctx->fuse_p && !multi && G == 1 && n_halo == 0 && ctx->nfaults == 0 && !sr && !cheb && !ppcg;
  abft_vec* const p = R[0].p();
  abft_vec* const r = R[0].r();
  if (fused) {
    abft_vec ptmp = *p;
    fused = spmv_chunks(ctx, R[0].A, R[0].nchunks, &ptmp, R[0].w(), true, R[0].cnt, nullptr, s, nullptr, MODE_CORRECT,
                        0, reinterpret_cast<uint64_t*>(p->data), reinterpret_cast<uint64_t*>(r->data),
                        true) == ABFT_OK;
  }
  if (fused && ctx->p_alt_len < npad_ext) {
    cudaFree(ctx->p_alt);
    ctx->p_alt = nullptr;
    ctx->p_alt_len = 0;
    CUDA_TRY(cudaMalloc(&ctx->p_alt, sizeof(uint64_t) * npad_ext));
    ctx->p_alt_len = npad_ext;
  }
  uint64_t* const P[2] = {reinterpret_cast<uint64_t*>(p->data), ctx->p_alt};
  // peer-memory halos: calc_p stores p's boundary rows into the
  // neighbours' ghost rows and k_post_p raises their arrival flags; the SpMV's
  // halo step becomes a wait on this rank's flags.  Standard CG only, equal
  // strips, no fault schedule (an injected p fault must reach the ghost copy)
  bool peer = multi && d->peer_halo && d->nranks > 1 && n_halo > 0 && !sr && !cheb && !ppcg;
  for (int q = 0; q < nl && peer; q++) peer = R[q].ctx->nfaults == 0 && R[q].n == R[0].n;
  if (peer) {
    auto ext = [](abft_vec* v) { return reinterpret_cast<uint64_t*>(v->data); };
    for (int q = 0; q < nl; q++) {
      VecArgs& va = R[q].va;
      va.halo_n = n_halo;
      if (d->loopback) {
        va.halo_up = q > 0 ? ext(R[q - 1].p()) + n_halo + R[q - 1].n : nullptr;
        va.halo_dn = q < nl - 1 ? ext(R[q + 1].p()) : nullptr;
        va.sig_up = q > 0 ? d->flags + 2 * (q - 1) + 1 : nullptr;
        va.sig_dn = q < nl - 1 ? d->flags + 2 * (q + 1) : nullptr;
      } else {
        va.halo_up = d->rank > 0 ? d->peer_p[0] + n_halo + R[0].n : nullptr;
        va.halo_dn = d->rank < d->nranks - 1 ? d->peer_p[1] : nullptr;
        va.sig_up = d->rank > 0 ? d->peer_flag[0] : nullptr;
        va.sig_dn = d->rank < d->nranks - 1 ? d->peer_flag[1] : nullptr;
      }
    }
    // (ordered before any neighbour's first signal: that comes after the init
    // all-gather, which needs this rank)
    CUDA_TRY(cudaMemsetAsync(d->flags, 0, sizeof(int) * 2 * (d->loopback ? nl : 1), s));
  }
  // halo overlap: P > 1 and every chunk of every rank on the tiled kernel
  bool overlap = multi && d->nranks > 1 && n_halo > 0;
  for (int q = 0; q < nl && overlap; q++)
    overlap = spmv_chunks(R[q].ctx, R[q].A, R[q].nchunks, R[q].p(), R[q].w(), true, R[q].cnt, nullptr, s, nullptr,
                          MODE_CORRECT, 0, nullptr, nullptr, true) == ABFT_OK;
  (void)cudaGetLastError();

  CgState h{};
  h.tol = opts->tol;
  h.max_iters = opts->max_iters;
  h.abort_policy = opts->due_policy == 0 ? 1 : 0;
  h.dist = multi ? 1 : 0;
  h.fused = fused ? 1 : 0;
  h.pcg = ppcg ? 1 : 0;
  h.alpha_log = ctx->cg_log;
  h.beta_log = ctx->cg_log + CG_LOG;
  if (cheb) {   // host arithmetic, rounded as written
    h.ch_theta = (R[0].eigmax + R[0].eigmin) / 2.0;
    h.ch_delta = (R[0].eigmax - R[0].eigmin) / 2.0;
    h.ch_sigma = h.ch_theta / h.ch_delta;
    h.ch_rho = 1.0 / h.ch_sigma;
  }
  for (int q = 0; q < nl; q++) {
    count_launch(launch_set_state(h, R[q].ctx->state, s));
    CUDA_TRY(cudaMemsetAsync(R[q].ctx->due, 0, sizeof(int), s));
  }

  Prof prof{ctx, s};
  // O10 fault schedule: iteration-0 faults before init
  for (int q = 0; q < nl; q++)
    count_launch(launch_inject_sched(R[q].ctx->faults, R[q].ctx->nfaults, R[q].ctx->state, 0, s));
  // init (a2): w = A x0 ; r = b - w ; p = r ; rr0
  if ((e = halo_exchange(d, R, nl, 1, n_halo, s))) return e;
  prof.begin(0);
  for (int q = 0; q < nl; q++) {
    e = spmv_chunks(R[q].ctx, R[q].A, R[q].nchunks, R[q].x(), R[q].w(), false, R[q].cnt, nullptr, s, nullptr,
                    MODE_CORRECT, interval);
    if (e) return e;
  }
  prof.end();
  if (!cheb)
    for (int q = 0; q < nl; q++) count_launch(launch_init_r(R[q].va, scheme, s));
  // peer-memory halos: iteration 1's p (= r, written by init) reaches the
  // ghost rows by one copy exchange; from then on the neighbours' calc_p
  // stores them (the loop's wait then passes on flags >= 0 at iteration 1)
  if (peer && (e = halo_exchange(d, R, nl, 3, n_halo, s))) return e;
  if (cheb) {   // r = b - A u0; p = r/theta; u += p; rr0
    count_launch(launch_cheb(R[0].va, scheme, 1, 0.0, 0.0, 0.0, s));
    if ((e = finish_dot(R, nl, d, 8, s))) return e;
  } else if (sr) {
    // p = s = encoded +0.0, then w = A r with both dots (gamma = r.r, delta = w.r)
    for (int q = 0; q < nl; q++)
      for (abft_vec* v : {R[q].p(), R[q].s_vec}) {
        const int64_t np = vec_padded_len(v->n, scheme);
        CUDA_TRY(cudaMemsetAsync(v->data, 0, sizeof(uint64_t) * np, s));
        count_launch(launch_vec_encode(reinterpret_cast<uint64_t*>(v->data), v->n, np, scheme, s));
      }
    if ((e = halo_exchange(d, R, nl, 2, n_halo, s))) return e;
    for (int q = 0; q < nl; q++)
      if ((e = spmv_chunks(R[q].ctx, R[q].A, R[q].nchunks, R[q].r(), R[q].w(), 2, R[q].cnt, nullptr, s, nullptr)))
        return e;
    if ((e = finish_sr(R, nl, d, 7, s))) return e;
  } else if ((e = finish_dot(R, nl, d, 1, s))) {
    return e;
  }
  // PPCG's preconditioner z = M^-1 r: inner Chebyshev steps from z = 0
  auto apply_prec = [&](cudaStream_t ss) -> int {
    count_launch(launch_cheb(vpc, scheme, 3, 0.0, 0.0, pc_theta, ss));
    for (size_t j = 0; j < pc_alpha.size(); j++) {
      int e2 = spmv_chunks(ctx, R[0].A, R[0].nchunks, R[0].z, R[0].w(), 0, R[0].cnt, ctx->state, ss, nullptr);
      if (e2) return e2;
      count_launch(launch_cheb(vpc, scheme, 2, pc_alpha[j], pc_beta[j], pc_theta, ss));
    }
    return ABFT_OK;
  };
  if (ppcg) {   // z = M^-1 r0; rz = r.z; p = z
    if ((e = apply_prec(s))) return e;
    count_launch(launch_dot(vdot, scheme, s));
    if ((e = finish_dot(R, nl, d, 12, s))) return e;
    count_launch(launch_copy_running(reinterpret_cast<uint64_t*>(R[0].p()->data),
                                     reinterpret_cast<const uint64_t*>(R[0].z->data), npad_ext, ctx->state, s));
  }
  CUDA_TRY(cudaGetLastError());

  int poll = opts->poll_every > 0 ? opts->poll_every : 16;
  if (fused && (poll & 1)) poll += 1;  // graph replays then always start at an odd iteration (buffer parity)
  int64_t launched = 0;  // iterations issued so far (host); = device iterations until a stop
  // PDL between the iteration kernels (single GPU: the multi-rank loop has
  // exchange steps in between); off again on every exit from this function
  struct PdlGuard {
    explicit PdlGuard(bool on) { set_pdl(on); }
    ~PdlGuard() { set_pdl(false); }
  };
  const bool pdl_on = ctx->pdl && !multi;
  // the protected SpMV of one iteration, all ranks (halo first, or overlapped)
  // vi: the SpMV's input vector (3 = p; 2 = r for the single-reduction CG), dots 1 or 2
  // the p halo of an iteration's SpMV: copied (NCCL send/recv, loopback
  // copies) or, with peer-memory halos, already stored by the neighbours'
  // calc_p — then wait for their arrival flags (identical in every graph replay)
  auto halo_step = [&](int vi, cudaStream_t hs) -> int {
    if (peer && vi == 3) {
      for (int q = 0; q < nl; q++) {
        const bool up = d->loopback ? q > 0 : d->rank > 0;
        const bool dn = d->loopback ? q < nl - 1 : d->rank < d->nranks - 1;
        count_launch(launch_wait_halo(d->flags + (d->loopback ? 2 * q : 0), R[q].ctx->state, up, dn, hs));
      }
      return ABFT_OK;
    }
    return halo_exchange(d, R, nl, vi, n_halo, hs);
  };
  auto spmv_iter = [&](int64_t kk, cudaStream_t ss, int vi, int dots) -> int {
    int e2;
    if (fused) {
      abft_vec pprev = *p;
      pprev.data = reinterpret_cast<double*>(P[kk & 1]);
      return spmv_chunks(ctx, R[0].A, R[0].nchunks, &pprev, R[0].w(), true, R[0].cnt, ctx->state, ss, nullptr,
                         MODE_CORRECT, interval, P[(kk - 1) & 1], reinterpret_cast<uint64_t*>(r->data));
    }
    if (!overlap) {
      if ((e2 = halo_step(vi, ss))) return e2;
      for (int q = 0; q < nl; q++) {
        // standard CG: p was last written by calc_p (iteration 1: init), and
        // the kernel between it and this SpMV (k_post_p / the rr0 reduction)
        // writes no vector, so the window TMA may precede the PDL wait — unless
        // a fault-injection kernel sits between (PPCG's init copies p right
        // before iteration 1)
        const bool early = vi == 3 && !ppcg && (!pdl_on || R[q].ctx->nfaults == 0);
        if ((e2 = spmv_chunks(R[q].ctx, R[q].A, R[q].nchunks, R[q].v[vi], R[q].w(), dots, R[q].cnt, R[q].ctx->state,
                              ss, nullptr, MODE_CORRECT, interval, nullptr, nullptr, false, 0, early)))
          return e2;
      }
      return ABFT_OK;
    }
    // halo on the comm stream while the interior tile rows run on ss; then the boundary rows
    CUDA_TRY(cudaEventRecord(d->ev_fork, ss));
    CUDA_TRY(cudaStreamWaitEvent(d->comm_stream, d->ev_fork, 0));
    if ((e2 = halo_step(vi, d->comm_stream))) return e2;
    CUDA_TRY(cudaEventRecord(d->ev_join, d->comm_stream));
    for (int part = 1; part <= 2; part++) {
      if (part == 2) CUDA_TRY(cudaStreamWaitEvent(ss, d->ev_join, 0));
      for (int q = 0; q < nl; q++)
        if ((e2 = spmv_chunks(R[q].ctx, R[q].A, R[q].nchunks, R[q].v[vi], R[q].w(), dots, R[q].cnt, R[q].ctx->state,
                              ss, nullptr, MODE_CORRECT, interval, nullptr, nullptr, false, part)))
          return e2;
    }
    return ABFT_OK;
  };
  // k iterations of (a3)..(a5) + the DUE/convergence logic, all device-side
  auto issue = [&](int64_t k, cudaStream_t ss) -> int {
    PdlGuard pg(pdl_on);
    prof.s = ss;
    for (int64_t it = 0; it < k; it++) {
      int e2;
      // fused: iteration kk's p lives in P[(kk-1) & 1], its predecessor in P[kk & 1]
      const int64_t kk = launched + it + 1;
      for (int q = 0; q < nl; q++)   // O10: faults of this iteration, before its SpMV
        count_launch(launch_inject_sched(R[q].ctx->faults, R[q].ctx->nfaults, R[q].ctx->state, 1, ss));
      if (cheb) {   // w = A u; r = b - w, p, u; r.r and the step coefficients
        prof.begin(0);
        e2 = spmv_chunks(ctx, R[0].A, R[0].nchunks, R[0].x(), R[0].w(), 0, R[0].cnt, ctx->state, ss, nullptr);
        prof.end();
        if (e2) return e2;
        prof.begin(1);
        count_launch(launch_cheb(R[0].va, scheme, 0, 0.0, 0.0, 0.0, ss));
        prof.end();
        prof.begin(3);
        if ((e2 = finish_dot(R, nl, d, 9, ss))) return e2;
        prof.end();
        continue;
      }
      if (sr) {   // update, then w = A r with both dots, then the one reduction (+ all-gather)
        prof.begin(1);
        for (int q = 0; q < nl; q++) count_launch(launch_calc_sr(R[q].va_sr, scheme, ss));
        prof.end();
        prof.begin(0);
        e2 = spmv_iter(kk, ss, 2, 2);
        prof.end();
        if (e2) return e2;
        prof.begin(3);
        if ((e2 = finish_sr(R, nl, d, 6, ss))) return e2;
        prof.end();
        continue;
      }
      prof.begin(0);
      e2 = spmv_iter(kk, ss, 3, 1);
      prof.end();
      if (e2) return e2;
      prof.begin(3);
      if ((e2 = finish_dot(R, nl, d, 2, ss))) return e2;
      prof.end();
      prof.begin(1);
      for (int q = 0; q < nl; q++) {
        VecArgs vu = R[q].va;
        if (fused) vu.p = P[(kk - 1) & 1] + n_halo;
        count_launch(launch_calc_ur(vu, scheme, ss));
      }
      prof.end();
      prof.begin(3);
      if ((e2 = finish_dot(R, nl, d, 3, ss))) return e2;
      prof.end();
      if (ppcg) {   // z = M^-1 r; beta = (r.z)'/(r.z); p = z + beta p
        prof.begin(2);
        if ((e2 = apply_prec(ss))) return e2;
        count_launch(launch_dot(vdot, scheme, ss));
        prof.end();
        prof.begin(3);
        if ((e2 = finish_dot(R, nl, d, 11, ss))) return e2;
        prof.end();
        prof.begin(2);
        count_launch(launch_calc_p(vcp, scheme, ss));
        prof.end();
      } else if (!fused) {
        prof.begin(2);
        for (int q = 0; q < nl; q++) count_launch(launch_calc_p(R[q].va, scheme, ss));
        prof.end();
      }
      if (multi && h.abort_policy) {   // DUE consensus: every rank stops after the same iteration
        for (int q = 0; q < nl; q++) count_launch(launch_pack_due(R[q].sendbuf, R[q].ctx->due, ss));
        if ((e2 = allgather_pairs(d, ss))) return e2;
        for (int q = 0; q < nl; q++)
          count_launch(launch_due_combine(R[q].gathered, d->nranks, R[q].ctx->state, R[q].ctx->due, ss));
      }
    }
    CUDA_TRY(cudaGetLastError());
    return ABFT_OK;
  };
  // CUDA graph of `poll` iterations (all local ranks, exchange steps included):
  // one launch per poll, no per-kernel CPU launch cost; kernels read
  // alpha/beta/stop from device state.
  cudaGraphExec_t gexec = nullptr;
  struct GraphGuard {
    cudaGraphExec_t& g;
    ~GraphGuard() { if (g) cudaGraphExecDestroy(g); }
  } gguard{gexec};
  std::vector<std::pair<int, int>> gmarks;
  uint64_t glaunches = 0;
  // (profiling brackets kernels with events, which are not timeable inside a
  // graph replay: profiled solves launch kernels directly)
  const bool graphs = ctx->use_graphs && ctx->profile == 0;
  bool last_graph = false;
  for (;;) {
    CUDA_TRY(cudaMemcpyAsync(ctx->h_state, ctx->state, sizeof(CgState), cudaMemcpyDeviceToHost, s));
    CUDA_TRY(cudaStreamSynchronize(s));
    if (last_graph) {  // the graph's event nodes were re-recorded by this replay
      prof.marks = gmarks;
      prof.harvest(true);
      prof.marks.clear();
    } else {
      prof.harvest();
    }
    last_graph = false;
    if (ctx->h_state->stop || launched >= opts->max_iters) break;
    int64_t k = opts->max_iters - launched;
    if (k > poll) k = poll;
    if (graphs && k == poll) {
      if (!gexec) {
        prof.harvest();  // start the graph's marks from a clean list
        const uint64_t l0 = g_launches.load();
        // capture on the context's private stream (the caller's may be the
        // legacy default stream, which cannot be captured); replay on `s`
        if (!ctx->cap_stream) CUDA_TRY(cudaStreamCreateWithFlags(&ctx->cap_stream, cudaStreamNonBlocking));
        cudaGraph_t graph = nullptr;
        CUDA_TRY(cudaStreamBeginCapture(ctx->cap_stream, cudaStreamCaptureModeThreadLocal));
        e = issue(k, ctx->cap_stream);
        cudaError_t ce = cudaStreamEndCapture(ctx->cap_stream, &graph);
        prof.s = s;
        if (e) {
          if (graph) cudaGraphDestroy(graph);
          return e;
        }
        if (ce != cudaSuccess) return fail(ABFT_E_CUDA, "graph capture: %s", cudaGetErrorString(ce));
        cudaError_t ie = cudaGraphInstantiate(&gexec, graph, 0);
        cudaGraphDestroy(graph);
        if (ie != cudaSuccess) return fail(ABFT_E_CUDA, "graph instantiate: %s", cudaGetErrorString(ie));
        glaunches = g_launches.load() - l0;
        g_launches.fetch_sub(glaunches);  // counted per replay below
        gmarks = prof.marks;
      }
      prof.marks.clear();
      CUDA_TRY(cudaGraphLaunch(gexec, s));
      count_launch((int)glaunches);
      last_graph = true;
    } else {
      if ((e = issue(k, s))) return e;
    }
    launched += k;
  }
  // per-rank states (identical control decisions on every rank)
  std::vector<CgState> hs(nl);
  hs[0] = *ctx->h_state;
  for (int q = 1; q < nl; q++) {
    CUDA_TRY(cudaMemcpyAsync(ctx->h_state, R[q].ctx->state, sizeof(CgState), cudaMemcpyDeviceToHost, s));
    CUDA_TRY(cudaStreamSynchronize(s));
    hs[q] = *ctx->h_state;
  }
  if (fused) {
    // the final p back into the caller's buffer, then the calc_p the unfused
    // order runs before an abort / max_iters stop (state.pending_p)
    if (hs[0].iters >= 1 && ((hs[0].iters - 1) & 1))
      CUDA_TRY(cudaMemcpyAsync(p->data, ctx->p_alt, sizeof(uint64_t) * npad_ext, cudaMemcpyDeviceToDevice, s));
    if (hs[0].pending_p) {
      CgState t{};
      t.beta = hs[0].beta;
      t.max_iters = 0x7FFFFFFF;
      count_launch(launch_set_state(t, ctx->state, s));
      VecArgs vp = R[0].va;
      count_launch(launch_calc_p(vp, scheme, s));
      CUDA_TRY(cudaStreamSynchronize(s));
    }
  }
  for (int q = 0; q < nl; q++) {
    res[q].iters = hs[q].iters;
    res[q].rr0 = hs[q].rr0;
    res[q].rrn = hs[q].rrn;
    res[q].status = hs[q].stop ? hs[q].status : (opts->max_iters > 0 ? ABFT_E_NOT_CONVERGED : ABFT_OK);
  }
  // interval mode: detection-only integrity check of the whole matrix when the
  // last access (= iteration count) was not a checked one
  if (interval && hs[0].iters % interval != 0) {
    int any = 0;
    for (int q = 0; q < nl; q++) {
      CUDA_TRY(cudaMemsetAsync(R[q].ctx->due, 0, sizeof(int), s));
      for (int c = 0; c < R[q].nchunks; c++)
        count_launch(launch_check_csr(&R[q].A[c], R[q].cnt, R[q].ctx->due, 2, s));
    }
    if (multi) {
      for (int q = 0; q < nl; q++) count_launch(launch_pack_due(R[q].sendbuf, R[q].ctx->due, s));
      if ((e = allgather_pairs(d, s))) return e;
      std::vector<double> g(GATHER_W * (size_t)d->nranks);
      CUDA_TRY(cudaMemcpyAsync(g.data(), d->gathered, sizeof(double) * g.size(), cudaMemcpyDeviceToHost, s));
      CUDA_TRY(cudaStreamSynchronize(s));
      for (int rk = 0; rk < d->nranks; rk++) any |= g[GATHER_W * rk + 1] != 0.0;
    } else {
      CUDA_TRY(cudaMemcpyAsync(ctx->h_flags, ctx->due, sizeof(int), cudaMemcpyDeviceToHost, s));
      CUDA_TRY(cudaStreamSynchronize(s));
      any = ctx->h_flags[0] != 0;
    }
    if (any && h.abort_policy)
      for (int q = 0; q < nl; q++) if (res[q].status != ABFT_E_DUE) res[q].status = ABFT_E_DUE;
  }
  if (res[0].status != ABFT_OK)
    fail(res[0].status, "CG finished with status %d after %d iterations", res[0].status, res[0].iters);
  return res[0].status;
}

RankRun make_rank(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                  abft_vec* w, abft_counts* dcnt) {
  RankRun R;
  R.ctx = ctx;
  R.A = A;
  R.nchunks = nchunks;
  R.v[0] = b; R.v[1] = x; R.v[2] = r; R.v[3] = p; R.v[4] = w;
  R.cnt = reinterpret_cast<DevCounts*>(dcnt);
  return R;
}

int dist_streams(abft_dist* d) {
  CUDA_TRY(cudaStreamCreateWithFlags(&d->comm_stream, cudaStreamNonBlocking));
  CUDA_TRY(cudaEventCreateWithFlags(&d->ev_fork, cudaEventDisableTiming));
  CUDA_TRY(cudaEventCreateWithFlags(&d->ev_join, cudaEventDisableTiming));
  return ABFT_OK;
}

}  // namespace

extern "C" {

int abft_cg_solve(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                  abft_vec* w, const abft_cg_opts* opts, abft_cg_result* res, abft_counts* dcnt, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  RankRun R = make_rank(ctx, A, nchunks, b, x, r, p, w, dcnt);
  return cg_run(&R, 1, nullptr, 0, opts, res, (cudaStream_t)stream);
}

int abft_cg_solve_sr(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r,
                     abft_vec* p, abft_vec* w, abft_vec* sv, const abft_cg_opts* opts, abft_cg_result* res,
                     abft_counts* dcnt, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  if (!sv) return fail(ABFT_E_INVALID, "null vector s");
  RankRun R = make_rank(ctx, A, nchunks, b, x, r, p, w, dcnt);
  R.s_vec = sv;
  return cg_run(&R, 1, nullptr, 0, opts, res, (cudaStream_t)stream);
}

int abft_cheby_solve(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                     abft_vec* w, double eigmin, double eigmax, const abft_cg_opts* opts, abft_cg_result* res,
                     abft_counts* dcnt, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  RankRun R = make_rank(ctx, A, nchunks, b, x, r, p, w, dcnt);
  R.cheb = true;
  R.eigmin = eigmin;
  R.eigmax = eigmax;
  return cg_run(&R, 1, nullptr, 0, opts, res, (cudaStream_t)stream);
}

int abft_ppcg_solve(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                    abft_vec* w, abft_vec* z, abft_vec* rin, abft_vec* pin, double eigmin, double eigmax, int inner,
                    const abft_cg_opts* opts, abft_cg_result* res, abft_counts* dcnt, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  if (inner < 1 || inner > 64) return fail(ABFT_E_INVALID, "PPCG inner steps must be in [1, 64]");
  if (!z || !rin || !pin) return fail(ABFT_E_INVALID, "null PPCG vector");
  RankRun R = make_rank(ctx, A, nchunks, b, x, r, p, w, dcnt);
  R.ppcg_inner = inner;
  R.eigmin = eigmin;
  R.eigmax = eigmax;
  R.z = z;
  R.rin = rin;
  R.pin = pin;
  return cg_run(&R, 1, nullptr, 0, opts, res, (cudaStream_t)stream);
}

// Extreme eigenvalues of the symmetric tridiagonal (diag a[0..k), off-diagonal
// e[0..k-1)) by Sturm-sequence bisection (host, 64 halvings from the
// Gershgorin interval): TeaLeaf's Lanczos spectrum estimate.
static int sturm_count(const double* a, const double* e, int k, double x) {
  int neg = 0;
  double q = a[0] - x;
  if (q < 0) neg++;
  for (int i = 1; i < k; i++) {
    if (q == 0.0) q = 1e-300;
    q = (a[i] - x) - e[i - 1] * e[i - 1] / q;
    if (q < 0) neg++;
  }
  return neg;   // eigenvalues < x
}
static double tridiag_eig(const double* a, const double* e, int k, int which /* 0 min, 1 max */) {
  double lo = a[0], hi = a[0];
  for (int i = 0; i < k; i++) {
    const double rad = (i > 0 ? fabs(e[i - 1]) : 0.0) + (i + 1 < k ? fabs(e[i]) : 0.0);
    lo = fmin(lo, a[i] - rad);
    hi = fmax(hi, a[i] + rad);
  }
  const int target = which ? k - 1 : 0;   // index of the wanted eigenvalue
  for (int it = 0; it < 64; it++) {
    const double mid = 0.5 * (lo + hi);
    if (sturm_count(a, e, k, mid) > target) hi = mid;
    else lo = mid;
  }
  return 0.5 * (lo + hi);
}

int abft_cg_spectrum(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* b, abft_vec* x, abft_vec* r, abft_vec* p,
                     abft_vec* w, int steps, const abft_cg_opts* opts, double* eigmin, double* eigmax,
                     abft_cg_result* res, abft_counts* dcnt, void* stream) {
  if (!ctx || !opts || !eigmin || !eigmax || !res) return fail(ABFT_E_INVALID, "null argument");
  if (steps < 2 || steps > CG_LOG) return fail(ABFT_E_INVALID, "steps must be in [2, %d]", CG_LOG);
  abft_cg_opts o = *opts;
  o.max_iters = steps;
  o.tol = 0.0;
  RankRun R = make_rank(ctx, A, nchunks, b, x, r, p, w, dcnt);
  int e = cg_run(&R, 1, nullptr, 0, &o, res, (cudaStream_t)stream);
  if (e != ABFT_OK && e != ABFT_E_NOT_CONVERGED) return e;
  const int k = ctx->h_state->iters;   // the solve's final state (read back by cg_run)
  if (k < 2) return fail(ABFT_E_SHAPE, "spectrum estimate needs >= 2 CG steps (got %d)", k);
  std::vector<double> lg(2 * CG_LOG);
  CUDA_TRY(cudaMemcpy(lg.data(), ctx->cg_log, sizeof(double) * 2 * CG_LOG, cudaMemcpyDeviceToHost));
  const double* al = lg.data();
  const double* bl = lg.data() + CG_LOG;
  std::vector<double> a(k), off(k);
  for (int j = 0; j < k; j++) {
    a[j] = 1.0 / al[j] + (j > 0 ? bl[j - 1] / al[j - 1] : 0.0);
    if (j + 1 < k) off[j] = sqrt(bl[j]) / al[j];
  }
  *eigmin = tridiag_eig(a.data(), off.data(), k, 0);
  *eigmax = tridiag_eig(a.data(), off.data(), k, 1);
  return ABFT_OK;
}

int abft_dist_get_unique_id(void* out128) {
  if (!out128) return fail(ABFT_E_INVALID, "null out");
  ncclUniqueId id;
  NCCL_TRY(ncclGetUniqueId(&id));
  memcpy(out128, &id, sizeof(id));
  return ABFT_OK;
}

int abft_dist_init(abft_dist** out, const void* uid, int rank, int nranks, int device) {
  if (!out || !uid || nranks < 1 || rank < 0 || rank >= nranks) return fail(ABFT_E_INVALID, "bad dist args");
  CUDA_TRY(cudaSetDevice(device));
  abft_dist* d = new abft_dist();
  d->rank = rank;
  d->nranks = nranks;
  d->device = device;
  ncclUniqueId id;
  memcpy(&id, uid, sizeof(id));
  ncclResult_t nr = ncclCommInitRank(&d->comm, nranks, id, rank);
  if (nr != ncclSuccess) {
    delete d;
    return fail(ABFT_E_NCCL, "ncclCommInitRank: %s", ncclGetErrorString(nr));
  }
  int e = dist_streams(d);
  if (!e && cudaMalloc(&d->sendbuf, sizeof(double) * GATHER_W) != cudaSuccess) e = fail(ABFT_E_CUDA, "cudaMalloc sendbuf");
  if (!e && cudaMalloc(&d->gathered, sizeof(double) * GATHER_W * nranks) != cudaSuccess)
    e = fail(ABFT_E_CUDA, "cudaMalloc gathered");
  if (!e && cudaMalloc(&d->flags, sizeof(int) * 2) != cudaSuccess) e = fail(ABFT_E_CUDA, "cudaMalloc flags");
  if (e) {
    abft_dist_destroy(d);
    return e;
  }
  *out = d;
  return ABFT_OK;
}

int abft_dist_init_loopback(abft_dist** out, int nranks, int device) {
  if (!out || nranks < 1 || nranks > 1024) return fail(ABFT_E_INVALID, "bad loopback args");
  CUDA_TRY(cudaSetDevice(device));
  abft_dist* d = new abft_dist();
  d->loopback = 1;
  d->nranks = nranks;
  d->device = device;
  int e = dist_streams(d);
  if (!e && cudaMalloc(&d->gathered, sizeof(double) * GATHER_W * nranks) != cudaSuccess)
    e = fail(ABFT_E_CUDA, "cudaMalloc gathered");
  if (!e && cudaMalloc(&d->flags, sizeof(int) * 2 * nranks) != cudaSuccess) e = fail(ABFT_E_CUDA, "cudaMalloc flags");
  if (e) {
    abft_dist_destroy(d);
    return e;
  }
  *out = d;
  return ABFT_OK;
}

int abft_dist_set_peer_halo(abft_dist* d, int enable, void* const* peer_p, int* const* peer_flag) {
  if (!d) return fail(ABFT_E_INVALID, "null dist");
  if (!enable) {
    d->peer_halo = 0;
    return ABFT_OK;
  }
  if (!d->loopback) {
    if (!peer_p || !peer_flag) return fail(ABFT_E_INVALID, "NCCL transport: the neighbours' p and flags are needed");
    const bool up = d->rank > 0, dn = d->rank < d->nranks - 1;
    if ((up && (!peer_p[0] || !peer_flag[0])) || (dn && (!peer_p[1] || !peer_flag[1])))
      return fail(ABFT_E_INVALID, "missing neighbour pointer");
    for (int k = 0; k < 2; k++) {
      d->peer_p[k] = reinterpret_cast<uint64_t*>(peer_p[k]);
      d->peer_flag[k] = peer_flag[k];
    }
  }
  d->peer_halo = 1;
  return ABFT_OK;
}

int abft_dist_flags(abft_dist* d, int** flags) {
  if (!d || !flags) return fail(ABFT_E_INVALID, "null dist/flags");
  *flags = d->flags;
  return ABFT_OK;
}

int abft_ipc_get_handle(const void* dev_ptr, void* handle, int64_t* offset) {
  if (!dev_ptr || !handle || !offset) return fail(ABFT_E_INVALID, "null argument");
  CUdeviceptr base = 0;
  size_t size = 0;
  cudaPointerAttributes at{};
  CUDA_TRY(cudaPointerGetAttributes(&at, dev_ptr));
  // the allocation's base address: IPC handles name whole allocations
  static PFN_cuMemGetAddressRange_v3020 range = [] {
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    return (cudaGetDriverEntryPoint("cuMemGetAddressRange", &p, cudaEnableDefault, &q) == cudaSuccess &&
            q == cudaDriverEntryPointSuccess)
               ? reinterpret_cast<PFN_cuMemGetAddressRange_v3020>(p)
               : static_cast<PFN_cuMemGetAddressRange_v3020>(nullptr);
  }();
  if (!range || range(&base, &size, reinterpret_cast<CUdeviceptr>(dev_ptr)) != CUDA_SUCCESS)
    return fail(ABFT_E_CUDA, "cuMemGetAddressRange failed");
  cudaIpcMemHandle_t h;
  CUDA_TRY(cudaIpcGetMemHandle(&h, reinterpret_cast<void*>(base)));
  memcpy(handle, &h, sizeof(h));
  *offset = (int64_t)(reinterpret_cast<CUdeviceptr>(dev_ptr) - base);
  return ABFT_OK;
}

int abft_ipc_open_handle(const void* handle, int64_t offset, void** dev_ptr) {
  if (!handle || !dev_ptr) return fail(ABFT_E_INVALID, "null argument");
  cudaIpcMemHandle_t h;
  memcpy(&h, handle, sizeof(h));
  void* base = nullptr;
  CUDA_TRY(cudaIpcOpenMemHandle(&base, h, cudaIpcMemLazyEnablePeerAccess));
  *dev_ptr = static_cast<char*>(base) + offset;
  return ABFT_OK;
}

int abft_ipc_close_handle(void* dev_ptr, int64_t offset) {
  if (!dev_ptr) return ABFT_OK;
  CUDA_TRY(cudaIpcCloseMemHandle(static_cast<char*>(dev_ptr) - offset));
  return ABFT_OK;
}

int abft_dist_destroy(abft_dist* d) {
  if (!d) return ABFT_OK;
  if (d->comm) ncclCommDestroy(d->comm);
  cudaFree(d->sendbuf);
  cudaFree(d->gathered);
  cudaFree(d->flags);
  if (d->ev_fork) cudaEventDestroy(d->ev_fork);
  if (d->ev_join) cudaEventDestroy(d->ev_join);
  if (d->comm_stream) cudaStreamDestroy(d->comm_stream);
  delete d;
  return ABFT_OK;
}

int abft_cg_solve_dist(abft_dist* d, abft_ctx* ctx, const abft_csr* A, int nchunks, int64_t n_halo, abft_vec* b,
                       abft_vec* x, abft_vec* r, abft_vec* p, abft_vec* w, const abft_cg_opts* opts,
                       abft_cg_result* res, abft_counts* dcnt, void* stream) {
  if (!d || !ctx) return fail(ABFT_E_INVALID, "null dist/ctx");
  if (d->loopback) return fail(ABFT_E_INVALID, "loopback transport: use abft_cg_solve_loopback");
  RankRun R = make_rank(ctx, A, nchunks, b, x, r, p, w, dcnt);
  return cg_run(&R, 1, d, n_halo, opts, res, (cudaStream_t)stream);
}

int abft_cg_solve_sr_dist(abft_dist* d, abft_ctx* ctx, const abft_csr* A, int nchunks, int64_t n_halo, abft_vec* b,
                          abft_vec* x, abft_vec* r, abft_vec* p, abft_vec* w, abft_vec* sv, const abft_cg_opts* opts,
                          abft_cg_result* res, abft_counts* dcnt, void* stream) {
  if (!d || !ctx) return fail(ABFT_E_INVALID, "null dist/ctx");
  if (d->loopback) return fail(ABFT_E_INVALID, "loopback transport: use abft_cg_solve_loopback_sr");
  RankRun R = make_rank(ctx, A, nchunks, b, x, r, p, w, dcnt);
  R.s_vec = sv;
  return cg_run(&R, 1, d, n_halo, opts, res, (cudaStream_t)stream);
}

int abft_cg_solve_loopback_sr(abft_dist* d, abft_ctx* const* ctxs, const abft_csr* const* A, const int* nchunks,
                              int64_t n_halo, abft_vec* const* vecs, const abft_cg_opts* opts, abft_cg_result* res,
                              abft_counts* const* dcnt, void* stream) {
  if (!d || !d->loopback) return fail(ABFT_E_INVALID, "abft_cg_solve_loopback_sr needs a loopback transport");
  if (!ctxs || !A || !nchunks || !vecs || !dcnt) return fail(ABFT_E_INVALID, "null per-rank arrays");
  std::vector<RankRun> R(d->nranks);
  for (int q = 0; q < d->nranks; q++) {
    abft_vec* const* v = vecs + 6 * q;
    R[q] = make_rank(ctxs[q], A[q], nchunks[q], v[0], v[1], v[2], v[3], v[4], dcnt[q]);
    R[q].s_vec = v[5];
  }
  return cg_run(R.data(), d->nranks, d, n_halo, opts, res, (cudaStream_t)stream);
}

int abft_cg_solve_loopback(abft_dist* d, abft_ctx* const* ctxs, const abft_csr* const* A, const int* nchunks,
                           int64_t n_halo, abft_vec* const* vecs, const abft_cg_opts* opts, abft_cg_result* res,
                           abft_counts* const* dcnt, void* stream) {
  if (!d || !d->loopback) return fail(ABFT_E_INVALID, "abft_cg_solve_loopback needs a loopback transport");
  if (!ctxs || !A || !nchunks || !vecs || !dcnt) return fail(ABFT_E_INVALID, "null per-rank arrays");
  std::vector<RankRun> R(d->nranks);
  for (int q = 0; q < d->nranks; q++) {
    abft_vec* const* v = vecs + 5 * q;
    R[q] = make_rank(ctxs[q], A[q], nchunks[q], v[0], v[1], v[2], v[3], v[4], dcnt[q]);
  }
  return cg_run(R.data(), d->nranks, d, n_halo, opts, res, (cudaStream_t)stream);
}

int abft_check_all(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* vecs, int nvec, int scrub,
                   abft_counts* dcnt, void* stream) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  cudaStream_t s = (cudaStream_t)stream;
  DevCounts* cnt = reinterpret_cast<DevCounts*>(dcnt);
  if (A && nchunks > 0) {
    int e = check_chunks(A, nchunks);
    if (e) return e;
    for (int c = 0; c < nchunks; c++) count_launch(launch_check_csr(&A[c], cnt, ctx->due, scrub, s));
  }
  for (int i = 0; i < nvec; i++) {
    int e = check_vec(&vecs[i], "vecs[i]");
    if (e) return e;
    count_launch(launch_vec_check(reinterpret_cast<uint64_t*>(vecs[i].data), vecs[i].n,
                                  vec_padded_len(vecs[i].n, vecs[i].scheme), vecs[i].scheme, nullptr, cnt, ctx->due,
                                  scrub, s));
  }
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

// a4 / a5 as single calls: a scratch CG state carries alpha / beta (never stops)
static int blas1_setup(abft_ctx* ctx, abft_vec* const* v, int nv, double alpha, double beta, VecArgs& va,
                       cudaStream_t s, int32_t iters = 0) {
  if (!ctx) return fail(ABFT_E_INVALID, "null ctx");
  const char* names[4] = {"x", "p", "r", "w"};
  for (int i = 0; i < nv; i++) {
    int e = check_vec(v[i], names[i]);
    if (e) return e;
    if (v[i]->scheme != v[0]->scheme || v[i]->n != v[0]->n) return fail(ABFT_E_INVALID, "vectors differ");
    for (int j = 0; j < i; j++) if (v[i]->data == v[j]->data) return fail(ABFT_E_INVALID, "vectors alias");
  }
  const int64_t n = v[0]->n, nrb = (n + 255) / 256;
  int e = ensure_partials(ctx, nrb);
  if (e) return e;
  CgState h{};
  h.alpha = alpha;
  h.beta = beta;
  h.max_iters = 0x7FFFFFFF;
  h.iters = iters;
  count_launch(launch_set_state(h, ctx->state, s));
  va = VecArgs{};
  va.n = n;
  va.npad = vec_padded_len(n, v[0]->scheme);
  va.partials = ctx->partials;
  va.due = ctx->due;
  va.state = ctx->state;
  va.crc = ctx->crc;
  return ABFT_OK;
}

int abft_calc_ur(abft_ctx* ctx, abft_vec* x, abft_vec* p, abft_vec* r, abft_vec* w, double alpha, double* rrn_out,
                 abft_counts* dcnt, void* stream) {
  cudaStream_t s = (cudaStream_t)stream;
  abft_vec* v[4] = {x, p, r, w};
  VecArgs va;
  int e = blas1_setup(ctx, v, 4, alpha, 0.0, va, s);
  if (e) return e;
  va.x = reinterpret_cast<uint64_t*>(x->data);
  va.p = reinterpret_cast<uint64_t*>(p->data);
  va.r = reinterpret_cast<uint64_t*>(r->data);
  va.w = reinterpret_cast<uint64_t*>(w->data);
  va.counts = reinterpret_cast<DevCounts*>(dcnt);
  count_launch(launch_calc_ur(va, x->scheme, s));
  if (rrn_out)
    count_launch(launch_reduce(ctx->partials, (x->n + 255) / 256, ctx->roots, ctx->ticket, 0, nullptr, rrn_out,
                               ctx->due, s));
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

int abft_calc_p(abft_ctx* ctx, abft_vec* p, abft_vec* r, double beta, abft_counts* dcnt, void* stream) {
  cudaStream_t s = (cudaStream_t)stream;
  abft_vec* v[2] = {p, r};
  VecArgs va;
  int e = blas1_setup(ctx, v, 2, 0.0, beta, va, s);
  if (e) return e;
  va.p = reinterpret_cast<uint64_t*>(p->data);
  va.r = reinterpret_cast<uint64_t*>(r->data);
  va.counts = reinterpret_cast<DevCounts*>(dcnt);
  count_launch(launch_calc_p(va, p->scheme, s));
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

int abft_calc_p_spmv(abft_ctx* ctx, const abft_csr* A, int nchunks, abft_vec* p_prev, abft_vec* r, double beta,
                     abft_vec* p_out, abft_vec* out, double* dot_out, abft_counts* dcnt, void* stream) {
  cudaStream_t s = (cudaStream_t)stream;
  abft_vec* v[4] = {p_prev, r, p_out, out};
  VecArgs va;
  int e = check_chunks(A, nchunks);
  if (e) return e;
  const int vs = p_prev->scheme;
  if (vec_padded_len(1, vs) != 1) return fail(ABFT_E_SHAPE, "fused calc_p + SpMV: vector scheme with group size > 1");
  // the kernel takes the fused branch when state.iters > 0
  if ((e = blas1_setup(ctx, v, 4, 0.0, beta, va, s, 1))) return e;
  DevCounts* cnt = reinterpret_cast<DevCounts*>(dcnt);
  uint64_t* pc = reinterpret_cast<uint64_t*>(p_out->data);
  uint64_t* rf = reinterpret_cast<uint64_t*>(r->data);
  if (spmv_chunks(ctx, A, nchunks, p_prev, out, true, cnt, nullptr, s, nullptr, MODE_CORRECT, 0, pc, rf,
                  true) != ABFT_OK)
    return fail(ABFT_E_SHAPE, "fused calc_p + SpMV needs the tiled stencil path for every chunk");
  int64_t nrb = 0;
  e = spmv_chunks(ctx, A, nchunks, p_prev, out, true, cnt, ctx->state, s, &nrb, MODE_CORRECT, 0, pc, rf);
  if (e) return e;
  if (dot_out) count_launch(launch_reduce(ctx->partials, nrb, ctx->roots, ctx->ticket, 0, nullptr, dot_out, ctx->due, s));
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

int abft_ctx_set_faults(abft_ctx* ctx, const abft_fault* faults, int nfaults, const abft_csr* A, int nchunks,
                        abft_vec* const* vecs) {
  if (!ctx || nfaults < 0 || (nfaults > 0 && (!faults || !A || nchunks <= 0 || !vecs)))
    return fail(ABFT_E_INVALID, "bad fault schedule arguments");
  std::vector<DevFault> h((size_t)nfaults);
  for (int i = 0; i < nfaults; i++) {
    const abft_fault& f = faults[i];
    if (f.iter < 0 || f.word < 0) return fail(ABFT_E_INVALID, "fault %d: negative iteration / word", i);
    const int wbits = (f.target == ABFT_F_COL || f.target == ABFT_F_ROWPTR) ? 32 : 64;
    if (f.bit < 0 || f.bit >= wbits) return fail(ABFT_E_INVALID, "fault %d: bit out of range", i);
    uint8_t* base = nullptr;
    int64_t limit = 0;
    if (f.target <= ABFT_F_ROWPTR) {
      if (f.chunk < 0 || f.chunk >= nchunks) return fail(ABFT_E_INVALID, "fault %d: bad chunk", i);
      const abft_csr& M = A[f.chunk];
      if (f.target == ABFT_F_VAL) { base = reinterpret_cast<uint8_t*>(M.val); limit = M.nnz; }
      else if (f.target == ABFT_F_COL) { base = reinterpret_cast<uint8_t*>(M.col); limit = M.nnz; }
      else { base = reinterpret_cast<uint8_t*>(M.rowptr); limit = rowptr_padded_len(M.nrows, M.rowptr_scheme); }
    } else if (f.target <= ABFT_F_W) {
      abft_vec* v = vecs[f.target - ABFT_F_B];
      if (!v || !v->data) return fail(ABFT_E_INVALID, "fault %d: null vector", i);
      base = reinterpret_cast<uint8_t*>(v->data);
      limit = vec_padded_len(v->n, v->scheme);
    } else {
      return fail(ABFT_E_INVALID, "fault %d: bad target", i);
    }
    if (f.word >= limit) return fail(ABFT_E_INVALID, "fault %d: word beyond the target", i);
    const int64_t byte = f.word * (wbits / 8) + (f.bit / 32) * 4;
    h[i].addr = reinterpret_cast<uint32_t*>(base + byte);
    h[i].mask = 1u << (f.bit % 32);
    h[i].iter = f.iter;
  }
  cudaFree(ctx->faults);
  ctx->faults = nullptr;
  ctx->nfaults = 0;
  if (nfaults > 0) {
    CUDA_TRY(cudaMalloc(&ctx->faults, sizeof(DevFault) * (size_t)nfaults));
    CUDA_TRY(cudaMemcpy(ctx->faults, h.data(), sizeof(DevFault) * (size_t)nfaults, cudaMemcpyHostToDevice));
  }
  ctx->nfaults = nfaults;
  return ABFT_OK;
}

int abft_inject_bitflip(abft_ctx* ctx, void* dev_base, uint64_t bit_offset, void* stream) {
  if (!ctx || !dev_base) return fail(ABFT_E_INVALID, "null ctx/base");
  count_launch(launch_inject(dev_base, bit_offset, (cudaStream_t)stream));
  CUDA_TRY(cudaGetLastError());
  return ABFT_OK;
}

int abft_counts_read(const abft_counts* dcnt, abft_counts* host_out, void* stream) {
  if (!dcnt || !host_out) return fail(ABFT_E_INVALID, "null counts");
  cudaStream_t s = (cudaStream_t)stream;
  CUDA_TRY(cudaMemcpyAsync(host_out, dcnt, sizeof(abft_counts) * ABFT_T_COUNT * ABFT_SCHEME_COUNT,
                           cudaMemcpyDeviceToHost, s));
  CUDA_TRY(cudaStreamSynchronize(s));
  return ABFT_OK;
}

int abft_counts_reset(abft_counts* dcnt, void* stream) {
  if (!dcnt) return fail(ABFT_E_INVALID, "null counts");
  CUDA_TRY(cudaMemsetAsync(dcnt, 0, sizeof(abft_counts) * ABFT_T_COUNT * ABFT_SCHEME_COUNT, (cudaStream_t)stream));
  return ABFT_OK;
}

}  // extern "C"
