/*
 * ssbgen.h — seeded, counter-based generator of dbgen-shaped Star Schema Benchmark
 * (SSB) columns. This is the ONE module shared by the oracle (oracle/) and the CUDA
 * path (paper_journals_pvldb_chrysogeloskaa19_b200/): it produces INPUTS only and
 * holds none of the method's arithmetic (no filter, join, group-by or aggregate).
 *
 * Every value is a pure function of (seed, table sizes, column, row), so the host
 * (ssbgen_host.c) and the device (ssbgen_cuda.cu) produce bit-identical columns and a
 * partition [row_begin, row_end) can be generated without the rest of the table.
 *
 * Distributions (the SSB spec's, [SSB-spec]; the paper only cites SSB, PAPER.md:1124-1125,
 * and never prints the schema — see DESIGN.md "Readings"):
 *   lo_orderdate      uniform day in 1992-01-01 .. 1998-08-02 (2,406 days), as yyyymmdd
 *   lo_quantity       U[1,50]            lo_discount U[0,10]
 *   lo_custkey        U[1,C]  lo_partkey U[1,P]  lo_suppkey U[1,S]   (every FK matches)
 *   lo_extendedprice  lo_quantity * retail(lo_partkey)      (TPC-H retail price, cents)
 *   lo_revenue        lo_extendedprice * (100 - lo_discount) / 100   (truncating)
 *   lo_supplycost     6 * retail(lo_partkey) / 10                    (truncating)
 *   customer/supplier nation U[0,24]; region = TPC-H map; city = nation*10 + U[0,9]
 *   part              mfgr U[0,4]; category = mfgr*5 + U[0,4]; brand1 = category*40 + U[0,39]
 *   date              the full calendar 1992-01-01 .. 1998-12-31 (2,557 rows)
 *   micro-benchmarks  mb_value U[0,2^20); mb_probekey U[1, 2*n_part]; mb_buildkey 2*row+1
 * Dictionary codes are order-preserving (alphabetical regions/nations, see ssbgen/__init__.py).
 */
#ifndef SSBGEN_H
#define SSBGEN_H
#include <stdint.h>

#if defined(__CUDACC__)
#define SSBGEN_FN __host__ __device__ static inline
#else
#define SSBGEN_FN static inline
#endif

#ifdef __cplusplus
extern "C" {
#endif

/* Column ids. Lineorder 0..8, date 16.., customer 32.., supplier 48.., part 64.. */
enum {
  SSB_LO_ORDERDATE = 0, SSB_LO_CUSTKEY = 1, SSB_LO_PARTKEY = 2, SSB_LO_SUPPKEY = 3,
  SSB_LO_QUANTITY = 4, SSB_LO_EXTENDEDPRICE = 5, SSB_LO_DISCOUNT = 6, SSB_LO_REVENUE = 7,
  SSB_LO_SUPPLYCOST = 8,
  /* §6.4 micro-benchmark inputs: a fact table
     of n_lineorder rows with a value column (SUM query) and a probe-key column (1:N join),
     and a build table of n_part rows whose keys are the odd numbers 1, 3, .., 2*n_part-1.
     Probe keys are uniform over [1, 2*n_part], so about half of them match one build key. */
  MB_VALUE = 9, MB_PROBEKEY = 10, MB_BUILDKEY = 68,
  SSB_D_DATEKEY = 16, SSB_D_YEAR = 17, SSB_D_YEARMONTHNUM = 18, SSB_D_WEEKNUMINYEAR = 19,
  SSB_D_DAYNUMINYEAR = 20, SSB_D_MONTHNUMINYEAR = 21,
  SSB_C_CUSTKEY = 32, SSB_C_CITY = 33, SSB_C_NATION = 34, SSB_C_REGION = 35,
  SSB_S_SUPPKEY = 48, SSB_S_CITY = 49, SSB_S_NATION = 50, SSB_S_REGION = 51,
  SSB_P_PARTKEY = 64, SSB_P_MFGR = 65, SSB_P_CATEGORY = 66, SSB_P_BRAND1 = 67
};

typedef struct {
  int64_t n_lineorder, n_customer, n_supplier, n_part, n_date;
} ssbgen_sizes;

#define SSBGEN_N_DATE 2557          /* 1992-01-01 .. 1998-12-31 */
#define SSBGEN_N_ORDERDAYS 2406     /* 1992-01-01 .. 1998-08-02 */
#define SSBGEN_EPOCH_1992 8035      /* days from 1970-01-01 to 1992-01-01 */

/* Independent random streams (one per random variable, not per column). */
enum {
  SSBGEN_ST_ORDERDAY = 1, SSBGEN_ST_CUSTKEY = 2, SSBGEN_ST_PARTKEY = 3, SSBGEN_ST_SUPPKEY = 4,
  SSBGEN_ST_QUANTITY = 5, SSBGEN_ST_DISCOUNT = 6,
  SSBGEN_ST_C_NATION = 17, SSBGEN_ST_C_CITY = 18, SSBGEN_ST_S_NATION = 19, SSBGEN_ST_S_CITY = 20,
  SSBGEN_ST_P_MFGR = 21, SSBGEN_ST_P_CAT = 22, SSBGEN_ST_P_BRAND = 23,
  SSBGEN_ST_MB_VALUE = 24, SSBGEN_ST_MB_PROBE = 25
};

SSBGEN_FN uint64_t ssbgen_splitmix64(uint64_t x) {
  uint64_t z = x + 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}

/* Uniform integer in [0, range) from stream `st`, counter `row`. */
SSBGEN_FN uint32_t ssbgen_uniform(uint64_t seed, int st, int64_t row, uint32_t range) {
  uint64_t v = ssbgen_splitmix64(seed ^ ((uint64_t)st << 56) ^ (uint64_t)row);
  return (uint32_t)(((v >> 32) * (uint64_t)range) >> 32);
}

/* Civil date (y, m, d) from days since 1970-01-01 (proleptic Gregorian). */
SSBGEN_FN void ssbgen_civil(int64_t z, int32_t* y, int32_t* m, int32_t* d) {
  z += 719468;
  int64_t era = (z >= 0 ? z : z - 146096) / 146097;
  int64_t doe = z - era * 146097;
  int64_t yoe = (doe - doe / 1460 + doe / 36524 - doe / 146096) / 365;
  int64_t yy = yoe + era * 400;
  int64_t doy = doe - (365 * yoe + yoe / 4 - yoe / 100);
  int64_t mp = (5 * doy + 2) / 153;
  int64_t dd = doy - (153 * mp + 2) / 5 + 1;
  int64_t mm = mp < 10 ? mp + 3 : mp - 9;
  *y = (int32_t)(yy + (mm <= 2));
  *m = (int32_t)mm;
  *d = (int32_t)dd;
}

SSBGEN_FN int ssbgen_is_leap(int32_t y) { return (y % 4 == 0 && y % 100 != 0) || y % 400 == 0; }

/* Days before month m (1-based) in a non-leap year, without a lookup table (device code
   keeps no local arrays): 0,31,59,90,120,151,181,212,243,273,304,334. */
SSBGEN_FN int32_t ssbgen_days_before_month(int32_t m) {
  return m <= 2 ? (m - 1) * 31 : (153 * (m - 3) + 2) / 5 + 59;
}

/* 1-based day number within the year. */
SSBGEN_FN int32_t ssbgen_daynuminyear(int32_t y, int32_t m, int32_t d) {
  return ssbgen_days_before_month(m) + d + ((m > 2 && ssbgen_is_leap(y)) ? 1 : 0);
}

/* yyyymmdd of day index `day` counted from 1992-01-01. */
SSBGEN_FN int32_t ssbgen_datekey(int64_t day) {
  int32_t y, m, d;
  ssbgen_civil(SSBGEN_EPOCH_1992 + day, &y, &m, &d);
  return y * 10000 + m * 100 + d;
}

/* TPC-H retail price of part `pk`, in cents. */
SSBGEN_FN int32_t ssbgen_retail(int64_t pk) {
  return (int32_t)(90000 + ((pk / 10) % 20001) + 100 * (pk % 1000));
}

/* Region of each nation code (nations alphabetical, regions alphabetical; TPC-H map):
   ALGERIA ARGENTINA BRAZIL CANADA CHINA EGYPT ETHIOPIA FRANCE GERMANY INDIA INDONESIA
   IRAN IRAQ JAPAN JORDAN KENYA MOROCCO MOZAMBIQUE PERU ROMANIA RUSSIA SAUDI ARABIA
   UNITED KINGDOM UNITED STATES VIETNAM -> 0111240332244200011334312, packed 3 bits/nation. */
SSBGEN_FN int32_t ssbgen_nation_region(int32_t nation) {
  const uint64_t lo = 0ull | 0ull << 0 | 1ull << 3 | 1ull << 6 | 1ull << 9 | 2ull << 12 |
                      4ull << 15 | 0ull << 18 | 3ull << 21 | 3ull << 24 | 2ull << 27 | 2ull << 30 |
                      4ull << 33 | 4ull << 36 | 2ull << 39 | 4ull << 42 | 0ull << 45 | 0ull << 48 |
                      0ull << 51 | 1ull << 54 | 3ull << 57 | 3ull << 60;  /* nations 0..20 */
  const uint64_t hi = 4ull << 0 | 3ull << 3 | 1ull << 6 | 2ull << 9;        /* nations 21..24 */
  return nation < 21 ? (int32_t)((lo >> (3 * nation)) & 7u) : (int32_t)((hi >> (3 * (nation - 21))) & 7u);
}

/* The independent random variables, each a pure function of (seed, row). */
SSBGEN_FN int32_t ssbgen_lo_partkey(uint64_t seed, const ssbgen_sizes* sz, int64_t row) {
  return 1 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_PARTKEY, row, (uint32_t)sz->n_part);
}
SSBGEN_FN int32_t ssbgen_lo_quantity(uint64_t seed, int64_t row) {
  return 1 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_QUANTITY, row, 50);
}
SSBGEN_FN int32_t ssbgen_lo_discount(uint64_t seed, int64_t row) {
  return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_DISCOUNT, row, 11);
}
SSBGEN_FN int32_t ssbgen_p_category(uint64_t seed, int64_t row) {
  return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_P_MFGR, row, 5) * 5 +
         (int32_t)ssbgen_uniform(seed, SSBGEN_ST_P_CAT, row, 5);
}

/* Value of column `col` at row `row` (0-based). Returns 0 for an unknown column.
   (No recursion and no local arrays: identical code runs on the host and the device.) */
SSBGEN_FN int32_t ssbgen_value(uint64_t seed, const ssbgen_sizes* sz, int col, int64_t row) {
  switch (col) {
    case SSB_LO_ORDERDATE:
      return ssbgen_datekey(ssbgen_uniform(seed, SSBGEN_ST_ORDERDAY, row, SSBGEN_N_ORDERDAYS));
    case SSB_LO_CUSTKEY:
      return 1 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_CUSTKEY, row, (uint32_t)sz->n_customer);
    case SSB_LO_PARTKEY:
      return ssbgen_lo_partkey(seed, sz, row);
    case SSB_LO_SUPPKEY:
      return 1 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_SUPPKEY, row, (uint32_t)sz->n_supplier);
    case SSB_LO_QUANTITY:
      return ssbgen_lo_quantity(seed, row);
    case SSB_LO_DISCOUNT:
      return ssbgen_lo_discount(seed, row);
    case SSB_LO_EXTENDEDPRICE:
    case SSB_LO_REVENUE:
    case SSB_LO_SUPPLYCOST: {
      const int64_t retail = ssbgen_retail(ssbgen_lo_partkey(seed, sz, row));
      if (col == SSB_LO_SUPPLYCOST) return (int32_t)(6 * retail / 10);
      const int64_t ext = (int64_t)ssbgen_lo_quantity(seed, row) * retail;
      if (col == SSB_LO_EXTENDEDPRICE) return (int32_t)ext;
      return (int32_t)(ext * (100 - ssbgen_lo_discount(seed, row)) / 100);
    }
    case SSB_D_DATEKEY: return ssbgen_datekey(row);
    case SSB_D_YEAR: return ssbgen_datekey(row) / 10000;
    case SSB_D_YEARMONTHNUM: return ssbgen_datekey(row) / 100;
    case SSB_D_MONTHNUMINYEAR: return (ssbgen_datekey(row) / 100) % 100;
    case SSB_D_DAYNUMINYEAR:
    case SSB_D_WEEKNUMINYEAR: {
      int32_t y, m, d;
      ssbgen_civil(SSBGEN_EPOCH_1992 + row, &y, &m, &d);
      const int32_t dn = ssbgen_daynuminyear(y, m, d);
      return col == SSB_D_DAYNUMINYEAR ? dn : dn / 7 + 1;
    }
    case SSB_C_CUSTKEY: case SSB_S_SUPPKEY: case SSB_P_PARTKEY:
      return (int32_t)(row + 1);
    case SSB_C_NATION: return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_NATION, row, 25);
    case SSB_C_REGION:
      return ssbgen_nation_region((int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_NATION, row, 25));
    case SSB_C_CITY:
      return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_NATION, row, 25) * 10 +
             (int32_t)ssbgen_uniform(seed, SSBGEN_ST_C_CITY, row, 10);
    case SSB_S_NATION: return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_S_NATION, row, 25);
    case SSB_S_REGION:
      return ssbgen_nation_region((int32_t)ssbgen_uniform(seed, SSBGEN_ST_S_NATION, row, 25));
    case SSB_S_CITY:
      return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_S_NATION, row, 25) * 10 +
             (int32_t)ssbgen_uniform(seed, SSBGEN_ST_S_CITY, row, 10);
    case SSB_P_MFGR: return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_P_MFGR, row, 5);
    case SSB_P_CATEGORY: return ssbgen_p_category(seed, row);
    case SSB_P_BRAND1:
      return ssbgen_p_category(seed, row) * 40 +
             (int32_t)ssbgen_uniform(seed, SSBGEN_ST_P_BRAND, row, 40);
    case MB_VALUE: return (int32_t)ssbgen_uniform(seed, SSBGEN_ST_MB_VALUE, row, 1u << 20);
    case MB_PROBEKEY:
      return 1 + (int32_t)ssbgen_uniform(seed, SSBGEN_ST_MB_PROBE, row, (uint32_t)(2 * sz->n_part));
    case MB_BUILDKEY: return (int32_t)(2 * row + 1);
    default: return 0;
  }
}

/* Number of rows of the table that owns `col`. */
SSBGEN_FN int64_t ssbgen_table_rows(const ssbgen_sizes* sz, int col) {
  if (col < 16) return sz->n_lineorder;
  if (col < 32) return sz->n_date;
  if (col < 48) return sz->n_customer;
  if (col < 64) return sz->n_supplier;
  return sz->n_part;
}

#ifdef __cplusplus
}
#endif
#endif /* SSBGEN_H */
