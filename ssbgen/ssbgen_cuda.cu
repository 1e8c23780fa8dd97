/* Device fill of SSB columns (see ssbgen.h): the same pure functions as the host fill, so
   columns generated in HBM are bit-identical to ssbgen_fill(). Input generation only. */
#include <cuda_runtime.h>
#include "ssbgen.h"

__global__ void ssbgen_fill_kernel(uint64_t seed, ssbgen_sizes sz, int col, int64_t row_begin,
                                   int64_t n, int32_t* __restrict__ out) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < n;
       i += (int64_t)gridDim.x * blockDim.x)
    out[i] = ssbgen_value(seed, &sz, col, row_begin + i);
}

/* Fills device buffer out[0..n) on `stream` (a cudaStream_t, may be NULL). Returns 0 or the
   cudaError_t of the launch; -1 on a bad argument. Asynchronous. */
extern "C" int ssbgen_fill_device(uint64_t seed, const ssbgen_sizes* sz, int col,
                                  int64_t row_begin, int64_t n, int32_t* out, void* stream) {
  if (!sz || row_begin < 0 || n < 0 || row_begin + n > ssbgen_table_rows(sz, col)) return -1;
  if (n == 0) return 0;
  int64_t blocks = (n + 255) / 256;
  if (blocks > 148 * 32) blocks = 148 * 32;
  ssbgen_fill_kernel<<<(unsigned)blocks, 256, 0, (cudaStream_t)stream>>>(seed, *sz, col, row_begin,
                                                                        n, out);
  return (int)cudaGetLastError();
}
