// Microbenchmark: per-SM issue throughput of the integer / FP64 instructions the
// ABFT codec is built from (POPC, LOP3, SHF, IMAD, PRMT, DFMA), plus streaming
// HBM read / copy bandwidth.  Used to size the codec's ALU budget.
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o pipes pipes.cu
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { printf("CUDA %s @%d\n", cudaGetErrorString(e), __LINE__); return 1; } } while (0)

constexpr int CH = 8;        // independent chains per thread
constexpr int ITERS = 4096;

template <int OP>
__global__ void __launch_bounds__(1024) k_pipe(uint32_t* out, unsigned long long* clk, uint32_t seed) {
  uint32_t x[CH];
  double d[CH];
#pragma unroll
  for (int i = 0; i < CH; i++) { x[i] = seed * (threadIdx.x + 7 * i + 1); d[i] = (double)x[i]; }
  __syncthreads();
  unsigned long long t0 = clock64();
  for (int it = 0; it < ITERS; it++) {
#pragma unroll
    for (int i = 0; i < CH; i++) {
      if (OP == 0) asm volatile("popc.b32 %0, %0;" : "+r"(x[i]));
      if (OP == 1) asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(x[i]) : "r"(x[(i + 1) % CH]), "r"(seed));
      if (OP == 2) asm volatile("shf.r.wrap.b32 %0, %0, %1, 5;" : "+r"(x[i]) : "r"(x[(i + 3) % CH]));
      if (OP == 3) asm volatile("mad.lo.u32 %0, %0, %1, %2;" : "+r"(x[i]) : "r"(seed), "r"(x[(i + 1) % CH]));
      if (OP == 4) asm volatile("prmt.b32 %0, %0, %1, 0x3120;" : "+r"(x[i]) : "r"(x[(i + 1) % CH]));
      if (OP == 5) asm volatile("fma.rn.f64 %0, %0, %0, %1;" : "+d"(d[i]) : "d"(d[(i + 1) % CH]));
      if (OP == 6) {  // LOP3 + POPC interleaved: do the pipes overlap?
        uint32_t y;
        asm volatile("popc.b32 %0, %1;" : "=r"(y) : "r"(x[i]));
        asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(x[i]) : "r"(y), "r"(seed));
      }
      if (OP == 7) {  // LOP3 + IMAD interleaved
        asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(x[i]) : "r"(x[(i + 1) % CH]), "r"(seed));
        asm volatile("mad.lo.u32 %0, %0, %1, %2;" : "+r"(x[(i + 4) % CH]) : "r"(seed), "r"(x[(i + 2) % CH]));
      }
      if (OP == 8) asm volatile("add.u32 %0, %0, %1;" : "+r"(x[i]) : "r"(x[(i + 1) % CH]));
      if (OP == 9) asm volatile("shl.b32 %0, %0, 3;" : "+r"(x[i]));
    }
  }
  unsigned long long t1 = clock64();
  uint32_t acc = 0;
#pragma unroll
  for (int i = 0; i < CH; i++) acc ^= x[i] ^ (uint32_t)(long long)d[i];
  out[blockIdx.x * blockDim.x + threadIdx.x] = acc;
  if (threadIdx.x == 0) clk[blockIdx.x] = t1 - t0;
}

__global__ void k_read(const int4* __restrict__ a, size_t n, int* out) {
  int acc = 0;
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n; i += (size_t)gridDim.x * blockDim.x) {
    int4 v = __ldg(a + i);
    acc ^= v.x ^ v.y ^ v.z ^ v.w;
  }
  if (acc == 0x12345678) out[0] = acc;
}
__global__ void k_copy(const int4* __restrict__ a, int4* __restrict__ b, size_t n) {
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n; i += (size_t)gridDim.x * blockDim.x) b[i] = a[i];
}

template <int OP>
int run(const char* name, int nsm, uint32_t* dout, unsigned long long* dclk, double ops_per_iter) {
  k_pipe<OP><<<nsm, 1024>>>(dout, dclk, 12345u);
  CK(cudaDeviceSynchronize());
  k_pipe<OP><<<nsm, 1024>>>(dout, dclk, 12345u);
  CK(cudaDeviceSynchronize());
  unsigned long long h[1024];
  CK(cudaMemcpy(h, dclk, nsm * sizeof(unsigned long long), cudaMemcpyDeviceToHost));
  double mean = 0;
  for (int i = 0; i < nsm; i++) mean += (double)h[i];
  mean /= nsm;
  double warp_ops = 32.0 * ITERS * CH * ops_per_iter;  // thread-ops per warp
  double per_sm_clk = warp_ops * 32 /* warps */ / mean;
  printf("%-10s %8.1f thread-ops/clk/SM\n", name, per_sm_clk);
  return 0;
}

int main() {
  int dev = 0, nsm = 0, clk = 0;
  CK(cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, dev));
  CK(cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, dev));
  printf("SMs %d, clock %d kHz\n", nsm, clk);
  uint32_t* dout; unsigned long long* dclk;
  CK(cudaMalloc(&dout, nsm * 1024 * 4));
  CK(cudaMalloc(&dclk, nsm * 8));
  run<0>("POPC", nsm, dout, dclk, 1);
  run<1>("LOP3", nsm, dout, dclk, 1);
  run<2>("SHF", nsm, dout, dclk, 1);
  run<3>("IMAD", nsm, dout, dclk, 1);
  run<4>("PRMT", nsm, dout, dclk, 1);
  run<5>("DFMA", nsm, dout, dclk, 1);
  run<6>("POPC+LOP3", nsm, dout, dclk, 2);
  run<7>("LOP3+IMAD", nsm, dout, dclk, 2);
  run<8>("IADD", nsm, dout, dclk, 1);
  run<9>("SHL", nsm, dout, dclk, 1);

  size_t bytes = (size_t)4 << 30;
  int4 *a, *b; int* o;
  CK(cudaMalloc(&a, bytes)); CK(cudaMalloc(&b, bytes)); CK(cudaMalloc(&o, 4));
  CK(cudaMemset(a, 1, bytes)); CK(cudaMemset(b, 0, bytes));
  size_t n = bytes / 16;
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  for (int grid_mul : {4, 8, 16, 32}) {
    float best_r = 1e9, best_c = 1e9;
    for (int rep = 0; rep < 5; rep++) {
      cudaEventRecord(e0); k_read<<<nsm * grid_mul, 256>>>(a, n, o); cudaEventRecord(e1); cudaEventSynchronize(e1);
      float ms; cudaEventElapsedTime(&ms, e0, e1); if (ms < best_r) best_r = ms;
      cudaEventRecord(e0); k_copy<<<nsm * grid_mul, 256>>>(a, b, n / 2); cudaEventRecord(e1); cudaEventSynchronize(e1);
      cudaEventElapsedTime(&ms, e0, e1); if (ms < best_c) best_c = ms;
    }
    printf("grid %3dxSM: read %.1f GB/s  copy(r+w) %.1f GB/s\n", grid_mul, bytes / best_r / 1e6, bytes / best_c / 1e6);
  }
  CK(cudaGetLastError());
  return 0;
}
