// Microbenchmark: codec fast-path throughput on sm_100a (codewords/clk/SM),
// register-resident data, for the layout-preserving variants the kernels may
// use.  Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -std=c++17
//              --expt-relaxed-constexpr -I../../paper_conf_cluster_pawelczakmpm17_b200/csrc -o codec codec.cu
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
#include "codec.cuh"

using namespace abft;
constexpr int ITERS = 2048;
constexpr int NW = 8;  // words in flight per thread

// subset-sum (left-shift) Moebius: R[i] = XOR_{j subset of i} D[j]
__device__ __forceinline__ uint32_t moeb_sub(uint32_t d) {
  d ^= (d << 1) & 0xAAAAAAAAu;
  d ^= (d << 2) & 0xCCCCCCCCu;
  d ^= (d << 4) & 0xF0F0F0F0u;
  d ^= (d << 8) & 0xFF00FF00u;
  d ^= (d << 16) & 0xFFFF0000u;
  return d;
}
__device__ __forceinline__ uint32_t moeb16x2(uint32_t x) {
  x ^= (x >> 1) & 0x55555555u;
  x ^= (x >> 2) & 0x33333333u;
  x ^= (x >> 4) & 0x0F0F0F0Fu;
  x ^= (x >> 8) & 0x00FF00FFu;
  return x;
}

template <int V>
__global__ void __launch_bounds__(512) k_codec(uint32_t* out, unsigned long long* clk, uint32_t seed) {
  uint32_t a[NW], b[NW], c[NW];
#pragma unroll
  for (int i = 0; i < NW; i++) { a[i] = seed * (threadIdx.x + 3 * i + 1); b[i] = a[i] * 0x9E3779B9u; c[i] = b[i] ^ 0x5bd1e995u; }
  uint32_t acc = 0;
  __syncthreads();
  unsigned long long t0 = clock64();
  for (int it = 0; it < ITERS; it++) {
    if (V == 0) {  // current V64 check
#pragma unroll
      for (int i = 0; i < NW; i++) acc |= v64_bad(a[i], b[i]);
    } else if (V == 1) {  // V64 with subset-sum Moebius (IMAD.SHL candidates)
#pragma unroll
      for (int i = 0; i < NW; i++) {
        uint32_t r = moeb_sub(v64_fold(a[i], b[i]));
        uint32_t s56 = (uint32_t)(__popc(b[i] ^ (a[i] & 0x80u)) | __popc(a[i] & 0x8Eu)) & 1u;
        acc |= (r & 0xE8808000u) | s56;
      }
    } else if (V == 2) {  // packed pairs (16-bit fold)
#pragma unroll
      for (int i = 0; i < NW; i += 2) {
        uint32_t da = v64_fold(a[i], b[i]), db = v64_fold(a[i + 1], b[i + 1]);
        uint32_t x = moeb16x2(__byte_perm(da, db, 0x5410) ^ __byte_perm(da, db, 0x7632));
        uint32_t p = (uint32_t)(__popc(da >> 16) | __popc(db >> 16) | __popc(b[i] ^ (a[i] & 0x80u)) | __popc(a[i] & 0x8Eu) |
                                __popc(b[i + 1] ^ (a[i + 1] & 0x80u)) | __popc(a[i + 1] & 0x8Eu));
        acc |= (x & 0x01170117u) | (p & 1u);
      }
    } else if (V == 3) {  // current E96 check
#pragma unroll
      for (int i = 0; i < NW; i++) acc |= e96_bad(a[i], b[i], c[i]);
    } else if (V == 4) {  // E96 packed pairs
#pragma unroll
      for (int i = 0; i < NW; i += 2) {
        uint32_t da = e96_fold(a[i], b[i], c[i]), db = e96_fold(a[i + 1], b[i + 1], c[i + 1]);
        uint32_t x = moeb16x2(__byte_perm(da, db, 0x5410) ^ __byte_perm(da, db, 0x7632));
        uint32_t p = (uint32_t)(__popc(da >> 16) | __popc(db >> 16) |
                                __popc(b[i] ^ (c[i] & 0x9F000000u)) | __popc((c[i] & 0x7FFFFFFFu) ^ (b[i] & 0x80000000u)) |
                                __popc(b[i + 1] ^ (c[i + 1] & 0x9F000000u)) |
                                __popc((c[i + 1] & 0x7FFFFFFFu) ^ (b[i + 1] & 0x80000000u)));
        acc |= (x & 0x01170117u) | (p & 1u);
      }
    } else if (V == 5) {  // V64 encode via LUT (constant-bank LUT stands in for smem)
#pragma unroll
      for (int i = 0; i < NW; i++) {
        uint64_t e = v64_encode_lut(mk64(a[i], b[i]), c_v64_lut.r);
        acc ^= lo32(e);
      }
    } else if (V == 6) {  // pure IMAD.SHL + LOP3 mix, independent chains
#pragma unroll
      for (int i = 0; i < NW; i++) {
        uint32_t t = a[i] * 8u;
        a[i] = (a[i] ^ (t & 0xF0F0F0F0u));
      }
    } else if (V == 7) {  // pure SHF + LOP3
#pragma unroll
      for (int i = 0; i < NW; i++) {
        uint32_t t = a[i] >> 3;
        a[i] = (a[i] ^ (t & 0x0F0F0F0Fu));
      }
    }
    // perturb inputs cheaply so nothing is loop-invariant
#pragma unroll
    for (int i = 0; i < NW; i++) { a[i] += it; }
  }
  unsigned long long t1 = clock64();
  out[blockIdx.x * blockDim.x + threadIdx.x] = acc ^ a[0];
  if (threadIdx.x == 0) clk[blockIdx.x] = t1 - t0;
}

template <int V>
void run(const char* name, int nsm, uint32_t* d, unsigned long long* c, double per_iter) {
  for (int rep = 0; rep < 2; rep++) k_codec<V><<<nsm * 2, 512>>>(d, c, 7u);
  cudaDeviceSynchronize();
  unsigned long long h[512];
  cudaMemcpy(h, c, sizeof(unsigned long long) * nsm * 2, cudaMemcpyDeviceToHost);
  double mean = 0;
  for (int i = 0; i < nsm * 2; i++) mean += h[i];
  mean /= nsm * 2;
  double items = 1024.0 * ITERS * per_iter;  // 2 blocks x 512 threads per SM
  printf("%-28s %7.2f items/clk/SM  (%.1f clk per warp-item)\n", name, items / mean, mean / (items / 32.0));
}

int main() {
  int nsm;
  cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
  uint32_t* d;
  unsigned long long* c;
  cudaMalloc(&d, nsm * 1024 * 4);
  cudaMalloc(&c, nsm * 2 * 8);
  run<0>("V64 check (SHF moebius)", nsm, d, c, NW);
  run<1>("V64 check (subset, SHL)", nsm, d, c, NW);
  run<2>("V64 check packed pairs", nsm, d, c, NW);
  run<3>("E96 check", nsm, d, c, NW);
  run<4>("E96 check packed pairs", nsm, d, c, NW);
  run<5>("V64 encode LUT", nsm, d, c, NW);
  run<6>("IMAD.SHL+LOP3 (ops=2)", nsm, d, c, NW);
  run<7>("SHF+LOP3 (ops=2)", nsm, d, c, NW);
  printf("%s\n", cudaGetErrorString(cudaGetLastError()));
  return 0;
}
