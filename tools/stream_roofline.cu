// Read-only streaming ceiling on this B200 (calibration for K1's roofline, not product code):
// sum 4 int32 columns of N rows with (a) plain 128-bit loads, grid-stride, U in flight per
// thread, and (b) cp.async.bulk tiles into a shared-memory ring (the K1 producer design),
// for several tile sizes / stage counts / CTAs per SM. Prints GB/s per variant.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o stream_roofline tools/stream_roofline.cu
#include <cstdio>
#include <cstdint>
#include <vector>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { printf("%s: %s\n", #x, cudaGetErrorString(e)); return 1; } } while (0)

template <int U>
__global__ void ldg_sum(const int4* __restrict__ a, const int4* __restrict__ b, const int4* __restrict__ c,
                        const int4* __restrict__ d, long long n4, unsigned long long* out) {
  long long acc = 0;
  const long long stride = (long long)gridDim.x * blockDim.x;
  long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x;
  for (; i + (U - 1) * stride < n4; i += U * stride) {
    int4 va[U], vb[U], vc[U], vd[U];
#pragma unroll
    for (int u = 0; u < U; ++u) {
      va[u] = __ldcs(a + i + u * stride); vb[u] = __ldcs(b + i + u * stride);
      vc[u] = __ldcs(c + i + u * stride); vd[u] = __ldcs(d + i + u * stride);
    }
#pragma unroll
    for (int u = 0; u < U; ++u)
      acc += va[u].x + vb[u].y + vc[u].z + vd[u].w + va[u].w + vb[u].z + vc[u].y + vd[u].x;
  }
  for (; i < n4; i += stride) {
    int4 va = a[i], vb = b[i], vc = c[i], vd = d[i];
    acc += va.x + vb.y + vc.z + vd.w;
  }
  if (acc == 0x7fffffff) atomicAdd(out, (unsigned long long)acc);
}

__device__ __forceinline__ uint32_t su32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }

__global__ void bulk_sum(const int* __restrict__ a, const int* __restrict__ b, const int* __restrict__ c,
                         const int* __restrict__ d, long long n, int tile, int stages, unsigned long long* out) {
  extern __shared__ __align__(128) unsigned char sm[];
  uint64_t* full = (uint64_t*)sm;
  uint64_t* empty = full + stages;
  int* buf = (int*)(sm + 256);
  const int cw = (blockDim.x / 32) - 1;
  const long long ntiles = (n + tile - 1) / tile;
  if (threadIdx.x == 0) {
    for (int s = 0; s < stages; ++s) {
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(su32(full + s)), "r"(1));
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(su32(empty + s)), "r"(cw));
    }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  const int warp = threadIdx.x / 32, lane = threadIdx.x % 32;
  if (warp == cw) {
    if (lane == 0) {
      uint64_t pol;
      asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
      int s = 0; uint32_t ph = 0; long long k = 0;
      for (long long t = blockIdx.x; t < ntiles; t += gridDim.x, ++k) {
        if (k >= stages) {
          uint32_t ok = 0;
          while (!ok) {
            asm volatile("{ .reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2; selp.u32 %0,1,0,p; }"
                         : "=r"(ok) : "r"(su32(empty + s)), "r"(ph ^ 1) : "memory");
          }
        }
        const uint32_t bytes = tile * 4;
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(su32(full + s)), "r"(bytes * 4) : "memory");
        const int* srcs[4] = {a, b, c, d};
        for (int col = 0; col < 4; ++col)
          asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], %4;"
                       ::"r"(su32(buf + ((size_t)s * 4 + col) * tile)), "l"(srcs[col] + t * tile), "r"(bytes),
                       "r"(su32(full + s)), "l"(pol) : "memory");
        if (++s == stages) { s = 0; ph ^= 1; }
      }
    }
    return;
  }
  long long acc = 0;
  int s = 0; uint32_t ph = 0;
  for (long long t = blockIdx.x; t < ntiles; t += gridDim.x) {
    asm volatile("{ .reg .pred p; W: mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1; @!p bra W; }"
                 ::"r"(su32(full + s)), "r"(ph) : "memory");
    const int* st = buf + (size_t)s * 4 * tile;
    for (int r = warp * 32 + lane; r < tile; r += cw * 32)
      acc += st[r] + st[tile + r] + st[2 * tile + r] + st[3 * tile + r];
    __syncwarp();
    if (lane == 0) asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(su32(empty + s)) : "memory");
    if (++s == stages) { s = 0; ph ^= 1; }
  }
  if (acc == 0x7fffffff) atomicAdd(out, (unsigned long long)acc);
}

int main() {
  const long long n = 60000000;  // SF10 lineorder rows
  int *a, *b, *c, *d;
  unsigned long long* out;
  CK(cudaMalloc(&a, n * 4)); CK(cudaMalloc(&b, n * 4)); CK(cudaMalloc(&c, n * 4)); CK(cudaMalloc(&d, n * 4));
  CK(cudaMalloc(&out, 8));
  CK(cudaMemset(a, 1, n * 4)); CK(cudaMemset(b, 2, n * 4)); CK(cudaMemset(c, 3, n * 4)); CK(cudaMemset(d, 4, n * 4));
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0); cudaEventCreate(&e1);
  const double bytes = 16.0 * n;
  auto timeit = [&](auto launch) {
    for (int i = 0; i < 3; ++i) launch();
    cudaEventRecord(e0);
    const int reps = 10;
    for (int i = 0; i < reps; ++i) launch();
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms = 0; cudaEventElapsedTime(&ms, e0, e1);
    return bytes / (ms / reps * 1e-3) / 1e9;
  };
  for (int occ : {2, 4, 8}) {
    const long long n4 = n / 4;
    double g1 = timeit([&] { ldg_sum<1><<<sms * occ, 256>>>((int4*)a, (int4*)b, (int4*)c, (int4*)d, n4, out); });
    double g2 = timeit([&] { ldg_sum<2><<<sms * occ, 256>>>((int4*)a, (int4*)b, (int4*)c, (int4*)d, n4, out); });
    double g4 = timeit([&] { ldg_sum<4><<<sms * occ, 256>>>((int4*)a, (int4*)b, (int4*)c, (int4*)d, n4, out); });
    printf("ldg_sum 256thr x %d CTA/SM: U1 %.0f  U2 %.0f  U4 %.0f GB/s\n", occ, g1, g2, g4);
  }
  for (int tile : {1024, 2048, 4096, 8192}) {
    for (int stages : {2, 3, 4, 6}) {
      for (int threads : {288, 544}) {
        size_t smem = 256 + (size_t)stages * 4 * tile * 4;
        if (smem > 220 * 1024) continue;
        cudaFuncSetAttribute(bulk_sum, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        int occ = 0;
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, bulk_sum, threads, smem);
        if (occ < 1) continue;
        double g = timeit([&] { bulk_sum<<<sms * occ, threads, smem>>>(a, b, c, d, n, tile, stages, out); });
        printf("bulk_sum tile %5d stages %d threads %3d (%d CTA/SM, %6zu B smem): %.0f GB/s\n", tile,
               stages, threads, occ, smem, g);
      }
    }
  }
  CK(cudaGetLastError());
  return 0;
}
