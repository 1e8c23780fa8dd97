/*
 * ssb_oracle.cpp — TEST INFRASTRUCTURE ONLY. A plain, slow, single-threaded evaluator of
 * the 13 Star Schema Benchmark queries. Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / --impl reference legs may load it; the product path never does.
 *
 * What it computes: each SSB query is an inner
 * equi-join of lineorder with its dimensions on FK = PK, conjunctive filters, GROUP BY and
 * an exact int64 SUM — the SQL definition [SSB-spec]. HetExchange's broadcast hash joins,
 * block routing and per-device partial aggregates merged by the union router
 * (§6.1, §3.1, Listing 1) change only
 * HOW that result is reached, never WHAT it is, so the oracle is the definition written
 * out: per lineorder row, look up every matching dimension row (a join, so a missing key
 * drops the row and a duplicate key multiplies it), test the WHERE clause, and accumulate
 * SUM and COUNT per group in a std::map keyed by the dictionary codes of the GROUP BY
 * columns. It shares no code with the CUDA path (no hash tables, no ranks, no radix).
 *
 * String literals of the SSB query texts are encoded by the oracle's own dictionary below
 * (order-preserving codes; tests check it agrees with the generator's dictionary).
 */
#include <algorithm>
#include <array>
#include <cstdint>
#include <cstring>
#include <map>
#include <stdexcept>
#include <string>
#include <unordered_map>
#include <vector>

extern "C" {
/* Column pointers of one SSB database (host memory, caller-owned). */
typedef struct {
  int64_t n_lo;
  const int32_t *lo_orderdate, *lo_custkey, *lo_partkey, *lo_suppkey, *lo_quantity,
      *lo_extendedprice, *lo_discount, *lo_revenue, *lo_supplycost;
  int64_t n_date;
  const int32_t *d_datekey, *d_year, *d_yearmonthnum, *d_weeknuminyear;
  int64_t n_cust;
  const int32_t *c_custkey, *c_city, *c_nation, *c_region;
  int64_t n_supp;
  const int32_t *s_suppkey, *s_city, *s_nation, *s_region;
  int64_t n_part;
  const int32_t *p_partkey, *p_mfgr, *p_category, *p_brand1;
} oracle_db;

/* One result row: GROUP BY codes in SELECT order (unused slots 0), SUM and COUNT(*). */
typedef struct {
  int32_t key[3];
  int32_t n_keys;
  int64_t sum;
  int64_t count;
} oracle_row;
}

namespace {

// ---- the oracle's own dictionary for SSB string literals [SSB-spec] -------------------
const char* kRegions[] = {"AFRICA", "AMERICA", "ASIA", "EUROPE", "MIDDLE EAST"};
const char* kNations[] = {"ALGERIA", "ARGENTINA", "BRAZIL", "CANADA", "CHINA", "EGYPT",
                          "ETHIOPIA", "FRANCE", "GERMANY", "INDIA", "INDONESIA", "IRAN",
                          "IRAQ", "JAPAN", "JORDAN", "KENYA", "MOROCCO", "MOZAMBIQUE",
                          "PERU", "ROMANIA", "RUSSIA", "SAUDI ARABIA", "UNITED KINGDOM",
                          "UNITED STATES", "VIETNAM"};

int32_t region(const std::string& s) {
  for (int i = 0; i < 5; ++i)
    if (s == kRegions[i]) return i;
  throw std::runtime_error("unknown region " + s);
}
int32_t nation(const std::string& s) {
  for (int i = 0; i < 25; ++i)
    if (s == kNations[i]) return i;
  throw std::runtime_error("unknown nation " + s);
}
// 'UNITED KI1': the first 9 characters of the nation name (space padded) plus one digit.
int32_t city(const std::string& s) {
  std::string prefix = s.substr(0, 9);
  int digit = s[9] - '0';
  for (int i = 0; i < 25; ++i) {
    std::string n = kNations[i];
    n.resize(9, ' ');
    if (n == prefix) return i * 10 + digit;
  }
  throw std::runtime_error("unknown city " + s);
}
// 'MFGR#m' / 'MFGR#mc' / 'MFGR#mcbb'
int32_t mfgr(const std::string& s) { return s[5] - '1'; }
int32_t category(const std::string& s) { return (s[5] - '1') * 5 + (s[6] - '1'); }
int32_t brand1(const std::string& s) { return category(s) * 40 + (std::stoi(s.substr(7)) - 1); }

// ---- dimension rows keyed by primary key (a join may match 0, 1 or several rows) ------
struct DateRow { int32_t year, yearmonthnum, weeknuminyear; };
struct CustRow { int32_t city, nation, region; };
struct SuppRow { int32_t city, nation, region; };
struct PartRow { int32_t mfgr, category, brand1; };

template <class R>
using Index = std::unordered_map<int32_t, std::vector<R>>;

template <class R>
const std::vector<R>& lookup(const Index<R>& idx, int32_t key) {
  static const std::vector<R> none;
  auto it = idx.find(key);
  return it == idx.end() ? none : it->second;
}

// The dimension indexes (built once per database) and the lineorder columns a query scans.
struct Indexes {
  Index<DateRow> date;
  Index<CustRow> cust;
  Index<SuppRow> supp;
  Index<PartRow> part;
  explicit Indexes(const oracle_db& db) {
    for (int64_t i = 0; i < db.n_date; ++i)
      date[db.d_datekey[i]].push_back({db.d_year[i], db.d_yearmonthnum[i], db.d_weeknuminyear[i]});
    for (int64_t i = 0; i < db.n_cust; ++i)
      cust[db.c_custkey[i]].push_back({db.c_city[i], db.c_nation[i], db.c_region[i]});
    for (int64_t i = 0; i < db.n_supp; ++i)
      supp[db.s_suppkey[i]].push_back({db.s_city[i], db.s_nation[i], db.s_region[i]});
    for (int64_t i = 0; i < db.n_part; ++i)
      part[db.p_partkey[i]].push_back({db.p_mfgr[i], db.p_category[i], db.p_brand1[i]});
  }
};
struct Db {
  const oracle_db& t;   // lineorder columns
  const Indexes* ix;    // dimension rows by primary key
};

using Key = std::array<int32_t, 3>;
struct Acc { int64_t sum = 0, count = 0; };
using Groups = std::map<Key, Acc>;

inline void add(Groups& g, Key k, int64_t v) {
  Acc& a = g[k];
  a.sum += v;
  a.count += 1;
}

// ---- the 13 SSB queries [SSB-spec], one function each, written as their SQL text -------
// Q1.x: select sum(lo_extendedprice*lo_discount) as revenue from lineorder, date
//       where lo_orderdate = d_datekey and <date pred> and lo_discount between .. and <qty pred>
void q1_1(const Db& db, int64_t b, int64_t e, Groups& g) {
  const oracle_db& t = db.t;
  for (int64_t i = b; i < e; ++i)
    for (const DateRow& d : lookup(db.ix->date, t.lo_orderdate[i]))
      if (d.year == 1993 && t.lo_discount[i] >= 1 && t.lo_discount[i] <= 3 && t.lo_quantity[i] < 25)
        add(g, {0, 0, 0}, (int64_t)t.lo_extendedprice[i] * t.lo_discount[i]);
}
void q1_2(const Db& db, int64_t b, int64_t e, Groups& g) {
  const oracle_db& t = db.t;
  for (int64_t i = b; i < e; ++i)
    for (const DateRow& d : lookup(db.ix->date, t.lo_orderdate[i]))
      if (d.yearmonthnum == 199401 && t.lo_discount[i] >= 4 && t.lo_discount[i] <= 6 &&
          t.lo_quantity[i] >= 26 && t.lo_quantity[i] <= 35)
        add(g, {0, 0, 0}, (int64_t)t.lo_extendedprice[i] * t.lo_discount[i]);
}
void q1_3(const Db& db, int64_t b, int64_t e, Groups& g) {
  const oracle_db& t = db.t;
  for (int64_t i = b; i < e; ++i)
    for (const DateRow& d : lookup(db.ix->date, t.lo_orderdate[i]))
      if (d.weeknuminyear == 6 && d.year == 1994 && t.lo_discount[i] >= 5 &&
          t.lo_discount[i] <= 7 && t.lo_quantity[i] >= 26 && t.lo_quantity[i] <= 35)
        add(g, {0, 0, 0}, (int64_t)t.lo_extendedprice[i] * t.lo_discount[i]);
}

// Q2.x: select sum(lo_revenue), d_year, p_brand1 from lineorder, date, part, supplier
//       where lo_orderdate = d_datekey and lo_partkey = p_partkey and lo_suppkey = s_suppkey
//       and <part pred> and <supplier pred> group by d_year, p_brand1 order by d_year, p_brand1
template <class PartPred, class SuppPred>
void q2(const Db& db, int64_t b, int64_t e, Groups& g, PartPred pp, SuppPred sp) {
  const oracle_db& t = db.t;
  for (int64_t i = b; i < e; ++i)
    for (const DateRow& d : lookup(db.ix->date, t.lo_orderdate[i]))
      for (const PartRow& p : lookup(db.ix->part, t.lo_partkey[i]))
        for (const SuppRow& s : lookup(db.ix->supp, t.lo_suppkey[i]))
          if (pp(p) && sp(s)) add(g, {d.year, p.brand1, 0}, t.lo_revenue[i]);
}
void q2_1(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t cat = category("MFGR#12"), reg = region("AMERICA");
  q2(db, b, e, g, [&](const PartRow& p) { return p.category == cat; },
     [&](const SuppRow& s) { return s.region == reg; });
}
void q2_2(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t lo = brand1("MFGR#2221"), hi = brand1("MFGR#2228"), reg = region("ASIA");
  q2(db, b, e, g, [&](const PartRow& p) { return p.brand1 >= lo && p.brand1 <= hi; },
     [&](const SuppRow& s) { return s.region == reg; });
}
void q2_3(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t br = brand1("MFGR#2239"), reg = region("EUROPE");
  q2(db, b, e, g, [&](const PartRow& p) { return p.brand1 == br; },
     [&](const SuppRow& s) { return s.region == reg; });
}

// Q3.x: select <c attr>, <s attr>, d_year, sum(lo_revenue) as revenue
//       from customer, lineorder, supplier, date where lo_custkey = c_custkey and
//       lo_suppkey = s_suppkey and lo_orderdate = d_datekey and <c pred> and <s pred> and
//       <date pred> group by <c attr>, <s attr>, d_year order by d_year asc, revenue desc
template <class CP, class SP, class DP, class CK, class SK>
void q3(const Db& db, int64_t b, int64_t e, Groups& g, CP cp, SP sp, DP dp, CK ck, SK sk) {
  const oracle_db& t = db.t;
  for (int64_t i = b; i < e; ++i)
    for (const CustRow& c : lookup(db.ix->cust, t.lo_custkey[i]))
      for (const SuppRow& s : lookup(db.ix->supp, t.lo_suppkey[i]))
        for (const DateRow& d : lookup(db.ix->date, t.lo_orderdate[i]))
          if (cp(c) && sp(s) && dp(d)) add(g, {ck(c), sk(s), d.year}, t.lo_revenue[i]);
}
void q3_1(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t asia = region("ASIA");
  q3(db, b, e, g, [&](const CustRow& c) { return c.region == asia; },
     [&](const SuppRow& s) { return s.region == asia; },
     [&](const DateRow& d) { return d.year >= 1992 && d.year <= 1997; },
     [](const CustRow& c) { return c.nation; }, [](const SuppRow& s) { return s.nation; });
}
void q3_2(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t us = nation("UNITED STATES");
  q3(db, b, e, g, [&](const CustRow& c) { return c.nation == us; },
     [&](const SuppRow& s) { return s.nation == us; },
     [&](const DateRow& d) { return d.year >= 1992 && d.year <= 1997; },
     [](const CustRow& c) { return c.city; }, [](const SuppRow& s) { return s.city; });
}
void q3_3(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t k1 = city("UNITED KI1"), k5 = city("UNITED KI5");
  q3(db, b, e, g, [&](const CustRow& c) { return c.city == k1 || c.city == k5; },
     [&](const SuppRow& s) { return s.city == k1 || s.city == k5; },
     [&](const DateRow& d) { return d.year >= 1992 && d.year <= 1997; },
     [](const CustRow& c) { return c.city; }, [](const SuppRow& s) { return s.city; });
}
void q3_4(const Db& db, int64_t b, int64_t e, Groups& g) {
  // d_yearmonth = 'Dec1997' is the month whose d_yearmonthnum is 199712.
  const int32_t k1 = city("UNITED KI1"), k5 = city("UNITED KI5");
  q3(db, b, e, g, [&](const CustRow& c) { return c.city == k1 || c.city == k5; },
     [&](const SuppRow& s) { return s.city == k1 || s.city == k5; },
     [&](const DateRow& d) { return d.yearmonthnum == 199712; },
     [](const CustRow& c) { return c.city; }, [](const SuppRow& s) { return s.city; });
}

// Q4.x: select d_year, <attrs>, sum(lo_revenue - lo_supplycost) as profit
//       from date, customer, supplier, part, lineorder where lo_custkey = c_custkey and
//       lo_suppkey = s_suppkey and lo_partkey = p_partkey and lo_orderdate = d_datekey and
//       <preds> group by d_year, <attrs> order by d_year, <attrs>
template <class Pred, class KeyF>
void q4(const Db& db, int64_t b, int64_t e, Groups& g, Pred pred, KeyF key) {
  const oracle_db& t = db.t;
  for (int64_t i = b; i < e; ++i)
    for (const DateRow& d : lookup(db.ix->date, t.lo_orderdate[i]))
      for (const CustRow& c : lookup(db.ix->cust, t.lo_custkey[i]))
        for (const SuppRow& s : lookup(db.ix->supp, t.lo_suppkey[i]))
          for (const PartRow& p : lookup(db.ix->part, t.lo_partkey[i]))
            if (pred(d, c, s, p))
              add(g, key(d, c, s, p), (int64_t)t.lo_revenue[i] - (int64_t)t.lo_supplycost[i]);
}
void q4_1(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t am = region("AMERICA"), m1 = mfgr("MFGR#1"), m2 = mfgr("MFGR#2");
  q4(db, b, e, g,
     [&](const DateRow&, const CustRow& c, const SuppRow& s, const PartRow& p) {
       return c.region == am && s.region == am && (p.mfgr == m1 || p.mfgr == m2);
     },
     [](const DateRow& d, const CustRow& c, const SuppRow&, const PartRow&) {
       return Key{d.year, c.nation, 0};
     });
}
void q4_2(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t am = region("AMERICA"), m1 = mfgr("MFGR#1"), m2 = mfgr("MFGR#2");
  q4(db, b, e, g,
     [&](const DateRow& d, const CustRow& c, const SuppRow& s, const PartRow& p) {
       return c.region == am && s.region == am && (d.year == 1997 || d.year == 1998) &&
              (p.mfgr == m1 || p.mfgr == m2);
     },
     [](const DateRow& d, const CustRow&, const SuppRow& s, const PartRow& p) {
       return Key{d.year, s.nation, p.category};
     });
}
void q4_3(const Db& db, int64_t b, int64_t e, Groups& g) {
  const int32_t am = region("AMERICA"), us = nation("UNITED STATES"), cat = category("MFGR#14");
  q4(db, b, e, g,
     [&](const DateRow& d, const CustRow& c, const SuppRow& s, const PartRow& p) {
       return c.region == am && s.nation == us && (d.year == 1997 || d.year == 1998) &&
              p.category == cat;
     },
     [](const DateRow& d, const CustRow&, const SuppRow& s, const PartRow& p) {
       return Key{d.year, s.city, p.brand1};
     });
}

struct QueryDef {
  const char* name;
  void (*run)(const Db&, int64_t, int64_t, Groups&);
  int n_keys;
  int order;  // 0: no group; 1: ORDER BY the group keys in SELECT order;
              // 2: Q3 "d_year asc, revenue desc" (d_year is key[2]); 3: Q2 (d_year, p_brand1)
};
const QueryDef kQueries[] = {
    {"q1.1", q1_1, 0, 0}, {"q1.2", q1_2, 0, 0}, {"q1.3", q1_3, 0, 0},
    {"q2.1", q2_1, 2, 1}, {"q2.2", q2_2, 2, 1}, {"q2.3", q2_3, 2, 1},
    {"q3.1", q3_1, 3, 2}, {"q3.2", q3_2, 3, 2}, {"q3.3", q3_3, 3, 2}, {"q3.4", q3_4, 3, 2},
    {"q4.1", q4_1, 2, 1}, {"q4.2", q4_2, 3, 1}, {"q4.3", q4_3, 3, 1},
};

int64_t run_query(const char* qname, const Indexes& ix, const oracle_db* db, int64_t row_begin,
                  int64_t row_end, oracle_row* out, int64_t cap);
}  // namespace

extern "C" {

/* Runs SSB query `qname` ("q1.1" .. "q4.3") over lineorder rows [row_begin, row_end) and the
   full dimension tables. Writes at most `cap` rows to `out` in ORDER BY order (Q3 ties on
   revenue broken by the group codes ascending, reading R8). A query without
   GROUP BY yields exactly one row (count 0 when nothing qualifies: SQL NULL). Returns the
   row count, -1 for an unknown query or bad range, -2 if cap is too small. */
int64_t oracle_ssb_query(const char* qname, const oracle_db* db, int64_t row_begin,
                         int64_t row_end, oracle_row* out, int64_t cap) {
  if (!db) return -1;
  const Indexes ix(*db);
  return run_query(qname, ix, db, row_begin, row_end, out, cap);
}

/* The same over a prebuilt index of the dimension tables (oracle_index_new), so that many
   lineorder chunks (e.g. SF1000 regenerated 100 M rows at a time, on several threads) are
   evaluated without rebuilding the dimension maps: `lo` supplies only the lineorder columns
   (its dimension fields are ignored). The index is read-only here and may be shared. */
int64_t oracle_ssb_query_idx(const char* qname, const void* index, const oracle_db* lo,
                             int64_t row_begin, int64_t row_end, oracle_row* out, int64_t cap) {
  if (!index) return -1;
  return run_query(qname, *static_cast<const Indexes*>(index), lo, row_begin, row_end, out, cap);
}

/* Builds the dimension indexes of `db` (its lineorder fields are ignored); caller frees. */
void* oracle_index_new(const oracle_db* db) { return db ? new Indexes(*db) : nullptr; }
void oracle_index_free(void* index) { delete static_cast<Indexes*>(index); }

}  // extern "C"

namespace {
int64_t run_query(const char* qname, const Indexes& ix, const oracle_db* db, int64_t row_begin,
                  int64_t row_end, oracle_row* out, int64_t cap) {
  if (!qname || !db || row_begin < 0 || row_end < row_begin || row_end > db->n_lo) return -1;
  const QueryDef* q = nullptr;
  for (const QueryDef& d : kQueries)
    if (std::strcmp(d.name, qname) == 0) q = &d;
  if (!q) return -1;
  const Db index{*db, &ix};
  Groups g;
  q->run(index, row_begin, row_end, g);
  std::vector<std::pair<Key, Acc>> rows(g.begin(), g.end());  // std::map: keys ascending
  if (q->n_keys == 0 && rows.empty()) rows.push_back({Key{0, 0, 0}, Acc{}});
  if (q->order == 2)
    std::stable_sort(rows.begin(), rows.end(), [](const auto& a, const auto& b) {
      if (a.first[2] != b.first[2]) return a.first[2] < b.first[2];
      return a.second.sum > b.second.sum;
    });
  if ((int64_t)rows.size() > cap) return -2;
  for (size_t i = 0; i < rows.size(); ++i) {
    for (int k = 0; k < 3; ++k) out[i].key[k] = rows[i].first[k];
    out[i].n_keys = q->n_keys;
    out[i].sum = rows[i].second.sum;
    out[i].count = rows[i].second.count;
  }
  return (int64_t)rows.size();
}
}  // namespace

extern "C" {

/* Encodes an SSB string literal with the oracle's own dictionary (kind: 0 region,
   1 nation, 2 city, 3 mfgr, 4 category, 5 brand1). Exposed so tests can check it agrees with
   the generator's dictionary. Returns -1 for an unknown literal. */
int32_t oracle_encode(int kind, const char* s) {
  try {
    switch (kind) {
      case 0: return region(s);
      case 1: return nation(s);
      case 2: return city(s);
      case 3: return mfgr(s);
      case 4: return category(s);
      case 5: return brand1(s);
    }
  } catch (...) {
  }
  return -1;
}
}
