// Micro-benchmark: random 4-byte lookups into a table split across a thread-block cluster's
// distributed shared memory (each CTA holds 1/C of it), vs the same table read from L2.
// Question: can a K1 stage-S map too large for one CTA's shared memory (e.g. the SF1000
// supplier bitmap, 250 KB) be probed from DSMEM at the rate K1 needs (~2 rows/cycle/SM)?
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o tools/dsmem_probe tools/dsmem_probe.cu
#include <cooperative_groups.h>
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
namespace cg = cooperative_groups;

__device__ __forceinline__ uint32_t hash32(uint32_t x) {
  x ^= x >> 16; x *= 0x85EBCA6Bu; x ^= x >> 13; x *= 0xC2B2AE35u; x ^= x >> 16; return x;
}

template <int C>
__global__ void __cluster_dims__(C, 1, 1) k_dsmem(const uint32_t* table, int words_per_cta, int iters,
                                                  unsigned long long* out) {
  extern __shared__ uint32_t slice[];
  cg::cluster_group cl = cg::this_cluster();
  const int rank = cl.block_rank();
  for (int i = threadIdx.x; i < words_per_cta; i += blockDim.x) slice[i] = table[rank * words_per_cta + i];
  cl.sync();
  const uint32_t total = (uint32_t)words_per_cta * C;
  uint32_t acc = 0, x = blockIdx.x * blockDim.x + threadIdx.x;
  for (int it = 0; it < iters; ++it) {
    uint32_t w[8];
#pragma unroll
    for (int k = 0; k < 8; ++k) {
      const uint32_t idx = hash32(x + k * 0x9E3779B9u + it * 8) % total;
      const int owner = idx / words_per_cta;
      uint32_t* p = cl.map_shared_rank(slice, owner);
      w[k] = p[idx - owner * words_per_cta];
    }
#pragma unroll
    for (int k = 0; k < 8; ++k) acc += w[k];
    x += 12345;
  }
  cl.sync();
  if (acc == 0x12345678u) out[0] = acc;
}

__global__ void k_l2(const uint32_t* table, uint32_t total, int iters, unsigned long long* out) {
  uint32_t acc = 0, x = blockIdx.x * blockDim.x + threadIdx.x;
  for (int it = 0; it < iters; ++it) {
    uint32_t w[8];
#pragma unroll
    for (int k = 0; k < 8; ++k) w[k] = __ldg(table + hash32(x + k * 0x9E3779B9u + it * 8) % total);
#pragma unroll
    for (int k = 0; k < 8; ++k) acc += w[k];
    x += 12345;
  }
  if (acc == 0x12345678u) out[0] = acc;
}

__global__ void k_local(const uint32_t* table, int words, int iters, unsigned long long* out) {
  extern __shared__ uint32_t slice[];
  for (int i = threadIdx.x; i < words; i += blockDim.x) slice[i] = table[i];
  __syncthreads();
  uint32_t acc = 0, x = blockIdx.x * blockDim.x + threadIdx.x;
  for (int it = 0; it < iters; ++it) {
    uint32_t w[8];
#pragma unroll
    for (int k = 0; k < 8; ++k) w[k] = slice[hash32(x + k * 0x9E3779B9u + it * 8) % (uint32_t)words];
#pragma unroll
    for (int k = 0; k < 8; ++k) acc += w[k];
    x += 12345;
  }
  if (acc == 0x12345678u) out[0] = acc;
}

template <int C>
void run_cluster(const uint32_t* d_table, int words_per_cta, int threads, int iters, int sms, unsigned long long* d_out) {
  const size_t smem = (size_t)words_per_cta * 4;
  cudaFuncSetAttribute(k_dsmem<C>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  int grid = (sms / C) * C;
  cudaLaunchConfig_t cfg{};
  cfg.gridDim = dim3(grid); cfg.blockDim = dim3(threads); cfg.dynamicSmemBytes = smem;
  int nclusters = 0;
  cudaOccupancyMaxActiveClusters(&nclusters, (void*)k_dsmem<C>, &cfg);
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
  k_dsmem<C><<<grid, threads, smem>>>(d_table, words_per_cta, iters, d_out);
  cudaEventRecord(a);
  k_dsmem<C><<<grid, threads, smem>>>(d_table, words_per_cta, iters, d_out);
  cudaEventRecord(b);
  cudaEventSynchronize(b);
  float ms; cudaEventElapsedTime(&ms, a, b);
  const double lookups = (double)grid * threads * iters * 8;
  printf("cluster %d: %d CTAs (max active clusters %d), table %d KB, %.3f ms, %.2f G lookups/s, %.3f lookups/cycle/SM (1.965 GHz), err=%s\n",
         C, grid, nclusters, C * words_per_cta * 4 / 1024, ms, lookups / ms / 1e6, lookups / (ms * 1e-3) / grid / 1.965e9,
         cudaGetErrorString(cudaGetLastError()));
}

int main() {
  int sms; cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  const int threads = 512, iters = 2000;
  const int words_total = 64 * 1024;  // 256 KB table (SF1000 supplier bitmap size)
  uint32_t* d_table; unsigned long long* d_out;
  cudaMalloc(&d_table, words_total * 4 * 2); cudaMalloc(&d_out, 8);
  cudaMemset(d_table, 1, words_total * 4 * 2);
  run_cluster<2>(d_table, words_total / 2, threads, iters, sms, d_out);   // 128 KB per CTA
  run_cluster<4>(d_table, words_total / 4, threads, iters, sms, d_out);   // 64 KB per CTA
  run_cluster<8>(d_table, words_total / 8, threads, iters, sms, d_out);   // 32 KB per CTA
  {  // same table from L2
    cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
    k_l2<<<sms, threads>>>(d_table, words_total, iters, d_out);
    cudaEventRecord(a);
    k_l2<<<sms, threads>>>(d_table, words_total, iters, d_out);
    cudaEventRecord(b); cudaEventSynchronize(b);
    float ms; cudaEventElapsedTime(&ms, a, b);
    const double lookups = (double)sms * threads * iters * 8;
    printf("L2 (256 KB table, ld.global.nc): %.3f ms, %.2f G lookups/s, %.3f lookups/cycle/SM\n", ms, lookups / ms / 1e6, lookups / (ms * 1e-3) / sms / 1.965e9);
  }
  {  // local shared memory (64 KB table) for reference
    const int w = 16 * 1024;
    cudaFuncSetAttribute(k_local, cudaFuncAttributeMaxDynamicSharedMemorySize, w * 4);
    cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
    k_local<<<sms, threads, w * 4>>>(d_table, w, iters, d_out);
    cudaEventRecord(a);
    k_local<<<sms, threads, w * 4>>>(d_table, w, iters, d_out);
    cudaEventRecord(b); cudaEventSynchronize(b);
    float ms; cudaEventElapsedTime(&ms, a, b);
    const double lookups = (double)sms * threads * iters * 8;
    printf("local smem (64 KB): %.3f ms, %.3f lookups/cycle/SM\n", ms, lookups / (ms * 1e-3) / sms / 1.965e9);
  }
  return 0;
}
