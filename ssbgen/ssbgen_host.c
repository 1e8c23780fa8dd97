/* Host fill of SSB columns (see ssbgen.h). Input generation only: no method arithmetic. */
#include "ssbgen.h"

/* Fills out[0..n) with column `col` rows [row_begin, row_begin+n). Returns 0, or -1 on a
   bad argument (unknown column, negative range, rows beyond the table). */
int ssbgen_fill(uint64_t seed, const ssbgen_sizes* sz, int col, int64_t row_begin, int64_t n,
                int32_t* out) {
  if (!sz || (n > 0 && !out) || row_begin < 0 || n < 0) return -1;
  if (row_begin + n > ssbgen_table_rows(sz, col)) return -1;
#pragma omp parallel for schedule(static)
  for (int64_t i = 0; i < n; ++i) out[i] = ssbgen_value(seed, sz, col, row_begin + i);
  return 0;
}
