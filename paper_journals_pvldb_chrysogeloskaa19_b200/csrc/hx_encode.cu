// hx_encode.cu — narrow column encodings ("narrower encodings"):
// frame of reference over the column's [min, max], stored as 1 or 2 unsigned bytes per value.
// K1 stages such columns at their width (fewer HBM bytes per row) and widens them in
// registers; nothing else changes what a query computes.
#include "hx_internal.cuh"

namespace hx {
namespace {

__global__ void k_min_max(const int32_t* v, int64_t n, int* out) {
  int lo = INT_MAX, hi = INT_MIN;
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x) {
    const int x = __ldg(v + i);
    lo = min(lo, x);
    hi = max(hi, x);
  }
  for (int o = 16; o > 0; o >>= 1) {
    lo = min(lo, __shfl_xor_sync(0xFFFFFFFFu, lo, o));
    hi = max(hi, __shfl_xor_sync(0xFFFFFFFFu, hi, o));
  }
  if ((threadIdx.x & 31) == 0) {
    atomicMin(out, lo);
    atomicMax(out + 1, hi);
  }
}

template <typename T>
__global__ void k_narrow(const int32_t* v, int64_t n, int32_t base, T* out) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
    out[i] = (T)(uint32_t)(__ldg(v + i) - base);
}

}  // namespace

int column_min_max(hx_ctx* ctx, const int32_t* v, int64_t n, int32_t* lo, int32_t* hi) {
  *lo = 0;
  *hi = 0;
  if (n == 0) return HX_OK;
  int* d = nullptr;
  HX_CK(cudaMallocAsync(reinterpret_cast<void**>(&d), 2 * sizeof(int), ctx->stream));
  const int init[2] = {INT_MAX, INT_MIN};
  HX_CK(cudaMemcpyAsync(d, init, sizeof(init), cudaMemcpyHostToDevice, ctx->stream));
  const int grid = (int)std::min<int64_t>((int64_t)ctx->n_sms * 4, (n + 255) / 256);
  k_min_max<<<grid, 256, 0, ctx->stream>>>(v, n, d);
  HX_CK_LAUNCH("k_min_max");
  ctx->launches += 1;
  int h[2];
  HX_CK(cudaMemcpyAsync(h, d, sizeof(h), cudaMemcpyDeviceToHost, ctx->stream));
  cudaFreeAsync(d, ctx->stream);
  HX_CK(cudaStreamSynchronize(ctx->stream));
  *lo = h[0];
  *hi = h[1];
  return HX_OK;
}

int column_narrow(hx_ctx* ctx, const int32_t* v, int64_t n, int32_t base, int width, void* out) {
  if (n == 0) return HX_OK;
  const int grid = (int)std::min<int64_t>((int64_t)ctx->n_sms * 4, (n + 255) / 256);
  if (width == 1)
    k_narrow<uint8_t><<<grid, 256, 0, ctx->stream>>>(v, n, base, static_cast<uint8_t*>(out));
  else
    k_narrow<uint16_t><<<grid, 256, 0, ctx->stream>>>(v, n, base, static_cast<uint16_t*>(out));
  HX_CK_LAUNCH("k_narrow");
  ctx->launches += 1;
  return HX_OK;
}

}  // namespace hx
