#include <cstdio>
#include <vector>
#include <cuda_runtime.h>
#include "../ssbgen/ssbgen.h"
__device__ __noinline__ int32_t city_noinline(uint64_t seed, int64_t i) {
  return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_NATION, i, 25) * 10 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_CITY, i, 10);
}
__global__ void fill_a(uint64_t seed, int64_t n, int32_t* out) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
    out[i] = (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_NATION, i, 25) * 10 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_CITY, i, 10);
}
__global__ void fill_b(uint64_t seed, int64_t n, int32_t* out) {
#pragma unroll 1
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
    out[i] = (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_NATION, i, 25) * 10 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_CITY, i, 10);
}
__global__ void fill_c(uint64_t seed, int64_t n, int32_t* out) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
    out[i] = city_noinline(seed, i);
}
__global__ void fill_d(uint64_t seed, int64_t n, int32_t* out) {  // 32-bit index
  for (int i = blockIdx.x * blockDim.x + threadIdx.x; i < n; i += gridDim.x * blockDim.x)
    out[i] = (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_NATION, i, 25) * 10 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_CITY, i, 10);
}
int main() {
  int64_t n = 3000000;
  int32_t* d; cudaMalloc(&d, n * 4);
  std::vector<int32_t> h(n);
  auto check = [&](const char* name, int grid, auto kern) {
    cudaMemset(d, 0xff, n * 4);
    kern<<<grid, 256>>>(42, n, d);
    cudaError_t e = cudaDeviceSynchronize();
    cudaMemcpy(h.data(), d, n * 4, cudaMemcpyDeviceToHost);
    int64_t bad = 0, first = -1;
    for (int64_t i = 0; i < n; ++i) {
      int32_t ref = (int32_t)ssbgen_uniform(42, SSBGEN_ST_C_NATION, i, 25) * 10 + (int32_t)ssbgen_uniform(42, SSBGEN_ST_C_CITY, i, 10);
      if (h[i] != ref) { if (first < 0) first = i; ++bad; }
    }
    printf("%s grid %d: %s bad %lld first %lld (got %d)\n", name, grid, cudaGetErrorString(e), (long long)bad, (long long)first, first >= 0 ? h[first] : 0);
  };
  for (int grid : {4736, 1}) { check("a", grid, fill_a); check("b", grid, fill_b); check("c", grid, fill_c); check("d", grid, fill_d); }
}
