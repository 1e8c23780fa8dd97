// Does the bulk-copy (TMA) engine read page-locked host memory through UVA on this GPU?
// Copies 64 KB host -> shared with cp.async.bulk, checks the values, reports the time.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__global__ void probe(const int* src, int n, int* out) {
  extern __shared__ __align__(128) int buf[];
  __shared__ __align__(8) unsigned long long bar;
  const unsigned sb = (unsigned)__cvta_generic_to_shared(&bar);
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(sb));
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(sb), "r"(n * 4) : "memory");
    asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];"
                 ::"r"((unsigned)__cvta_generic_to_shared(buf)), "l"(src + (size_t)blockIdx.x * n), "r"(n * 4), "r"(sb) : "memory");
  }
  asm volatile("{\n.reg .pred p;\nW:\nmbarrier.try_wait.parity.shared::cta.b64 p, [%0], 0;\n@!p bra W;\n}\n" ::"r"(sb) : "memory");
  int bad = 0;
  for (int i = threadIdx.x; i < n; i += blockDim.x) bad += buf[i] != (int)(blockIdx.x * n + i);
  if (bad) atomicAdd(out, bad);
}

int main() {
  const int n = 16384, blocks = 4096;  // 256 MB
  int* h = nullptr;
  if (cudaHostAlloc(&h, (size_t)n * blocks * 4, cudaHostAllocMapped) != cudaSuccess) return 2;
  for (size_t i = 0; i < (size_t)n * blocks; ++i) h[i] = (int)i;
  int* d = nullptr;
  cudaHostGetDevicePointer(&d, h, 0);
  int* out;
  cudaMalloc(&out, 4);
  cudaMemset(out, 0, 4);
  cudaFuncSetAttribute(probe, cudaFuncAttributeMaxDynamicSharedMemorySize, n * 4);
  probe<<<blocks, 256, n * 4>>>(d, n, out);
  cudaError_t e = cudaDeviceSynchronize();
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  cudaEventRecord(a);
  probe<<<blocks, 256, n * 4>>>(d, n, out);
  cudaEventRecord(b);
  cudaError_t e2 = cudaDeviceSynchronize();
  float ms = 0;
  cudaEventElapsedTime(&ms, a, b);
  int bad = -1;
  cudaMemcpy(&bad, out, 4, cudaMemcpyDeviceToHost);
  printf("uva bulk copy: %s / %s, mismatches %d, %.1f GB/s (host ptr %p dev ptr %p)\n", cudaGetErrorString(e),
         cudaGetErrorString(e2), bad, (double)n * blocks * 4 / (ms * 1e6), (void*)h, (void*)d);
  return (e == cudaSuccess && e2 == cudaSuccess && bad == 0) ? 0 : 1;
}
