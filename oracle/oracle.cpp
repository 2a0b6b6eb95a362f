/*
 * oracle/oracle.cpp — CPU ORACLE.  TEST INFRASTRUCTURE ONLY.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl
 * reference leg may load this library.  It shares no code, header, constant or
 * table with the CUDA path (paper_conf_ipps_awadapo20_b200/), and neither
 * imports the other.
 *
 * What it computes is the PLAIN DEFINITION of the paper's dynamic graph
 * (§II-A): a directed weighted graph G = (V, E, W) stored as
 * one adjacency map A_u : v -> w per vertex u ("one std::unordered_map per
 * vertex", BASELINE.json north_star).  Batches are applied one after another
 * (phase-concurrent model); inside a batch the oracle walks the
 * edges in array order.  No hashing into buckets, no slabs, no tombstones: the
 * hash-table machinery of §IV is what the GPU path does to reach this result
 * faster, so none of it appears here.
 *
 * Readings of the paper where it is silent are the DESIGN.md "Q" readings
 * (SURVEY.md §8(c) ambiguity register); each is cited at its use below.
 *
 * Pins (tests/test_oracle.py, -m "not gpu"): dense |V|x|V| adjacency-matrix
 * model on random op sequences, the north-star invariants,
 * triangle counts against closed forms / brute force / trace(A^3)/6, and the
 * hand-worked fixtures in tests/golden/.  Parity unpinned: only the choice
 * among intra-batch duplicate weights (Q1), which the oracle reports as a
 * candidate set instead of a single value.
 */
#include <algorithm>
#include <cstdint>
#include <cstring>
#include <thread>
#include <unordered_map>
#include <unordered_set>
#include <utility>
#include <vector>

namespace {

enum { ORC_OK = 0, ORC_ERR_INVALID_ARGUMENT = 1, ORC_ERR_VERTEX_OUT_OF_RANGE = 2 };

/* Q18: vertex IDs are u32 below 2^32-2 (the two top values are reserved). */
constexpr uint64_t kMaxVertices = 0xFFFFFFFEull;

/* A stored edge: its weight, plus the number of the insert batch that last wrote
 * it.  The stamp is bookkeeping for the Q1 candidate sets only (it tells a second
 * write of a key inside one batch from a first one); the graph is A_u : v -> w. */
struct Entry {
  uint32_t w;
  uint32_t batch;  // (mod 2^32: a stamp only has to differ from the current batch's)
};

inline uint64_t key_of(uint32_t u, uint32_t v) { return ((uint64_t)u << 32) | v; }

struct Oracle {
  uint64_t cap = 0;
  bool directed = true;
  unsigned T = 1;        // host threads; thread t owns the vertices u with u % T == t
  uint32_t batch = 0;    // insert batches applied so far (mod 2^32)
  std::vector<std::unordered_map<uint32_t, Entry>> A;  // A_u : v -> w
  /* Q1: keys (u,v) written >= 2 times by their most recent insert batch, with
   * the weights that batch carried for them (in batch order); any one of them is a
   * correct stored weight ("only the most recent edge ... will be stored",
   * P:L469-471, and a parallel batch has no order).  Sharded like the rows: the
   * set of key (u,v) lives in cand[u % T]. */
  std::vector<std::unordered_map<uint64_t, std::vector<uint32_t>>> cand;
};

inline bool in_range(const Oracle& g, const uint32_t* a, uint64_t n) {
  for (uint64_t i = 0; i < n; ++i)
    if ((uint64_t)a[i] >= g.cap) return false;
  return true;
}

/* Undirected mode: every edge op (u,v[,w]) is applied as (u,v[,w]) and (v,u[,w])
 * (P:L445-449). */
void expand(const Oracle& g, const uint32_t* s, const uint32_t* d, const uint32_t* w, uint64_t n,
            std::vector<uint32_t>& S, std::vector<uint32_t>& D, std::vector<uint32_t>& W) {
  S.assign(s, s + n);
  D.assign(d, d + n);
  W.resize(n);
  for (uint64_t i = 0; i < n; ++i) W[i] = w ? w[i] : 0u;  // Q27: no weights -> 0
  if (!g.directed) {
    S.insert(S.end(), d, d + n);
    D.insert(D.end(), s, s + n);
    for (uint64_t i = 0; i < n; ++i) W.push_back(w ? w[i] : 0u);
  }
}

/* Run f(t) for t = 0..T-1 on T threads (T = 1: inline).  Work partitioned by vertex
 * (u % T) keeps every vertex's ops in batch order on one thread. */
constexpr uint64_t kParallelMin = 1u << 15;  // smaller batches: one thread
inline unsigned threads_for(const Oracle& g, uint64_t work) { return work < kParallelMin ? 1u : g.T; }

template <typename F>
void parallel(unsigned T, F f) {
  if (T <= 1) {
    f(0u);
    return;
  }
  std::vector<std::thread> th;
  th.reserve(T);
  for (unsigned t = 0; t < T; ++t) th.emplace_back(f, t);
  for (auto& x : th) x.join();
}

}  // namespace

extern "C" {

void* orc_create(uint64_t num_vertices, int directed) {
  if (num_vertices > kMaxVertices) return nullptr;
  Oracle* g = new Oracle();
  g->cap = num_vertices;
  g->directed = directed != 0;
  g->A.resize(num_vertices);  // hints only affect performance: none taken
  g->cand.resize(1);
  return g;
}

/* Host threads used by the following calls (default 1).  Results do not depend on
 * it: each vertex's ops stay in batch order on one thread. */
int orc_set_threads(void* h, unsigned threads) {
  Oracle& g = *static_cast<Oracle*>(h);
  if (threads < 1 || threads > 256) return ORC_ERR_INVALID_ARGUMENT;
  std::vector<std::unordered_map<uint64_t, std::vector<uint32_t>>> c(threads);
  for (auto& shard : g.cand)
    for (auto& kv : shard) c[(kv.first >> 32) % threads].emplace(kv.first, std::move(kv.second));
  g.cand.swap(c);
  g.T = threads;
  return ORC_OK;
}

void orc_destroy(void* h) { delete static_cast<Oracle*>(h); }

uint64_t orc_num_vertices(void* h) { return static_cast<Oracle*>(h)->cap; }

/* Edge insertion, Alg. 1 P:L539-554 / §IV-C1 P:L451-481.
 *   - an out-of-range endpoint rejects the whole batch, graph unchanged (Q7);
 *   - self-loops are skipped (Alg1:L3);
 *   - replace semantics: an existing key gets the new weight, otherwise the pair
 *     is added (fn3 P:L235-236);
 *   - *n_added counts keys that were absent before the batch (exact degree
 *     maintenance);
 *   - Q1: the first write of a key in this batch clears its old candidate set; a
 *     second write makes {first weight, second weight} its candidates, later
 *     writes append. */
int orc_insert_edges(void* h, const uint32_t* src, const uint32_t* dst, const uint32_t* w,
                     uint64_t n, uint64_t* n_added) {
  Oracle& g = *static_cast<Oracle*>(h);
  if (n_added) *n_added = 0;
  if (n && (!src || !dst)) return ORC_ERR_INVALID_ARGUMENT;
  if (!in_range(g, src, n) || !in_range(g, dst, n)) return ORC_ERR_VERTEX_OUT_OF_RANGE;
  std::vector<uint32_t> S, D, W;
  expand(g, src, dst, w, n, S, D, W);
  const uint32_t b = ++g.batch;
  const unsigned P = threads_for(g, S.size());
  std::vector<uint64_t> added(P, 0);
  parallel(P, [&](unsigned t) {
    uint64_t a = 0;
    for (size_t i = 0; i < S.size(); ++i) {
      const uint32_t u = S[i], v = D[i];
      if (u % P != t) continue;                         // another thread's vertex
      if (u == v) continue;                             // Alg1:L3
      auto& cand = g.cand[u % g.T];
      auto& Au = g.A[u];
      auto it = Au.find(v);
      if (it == Au.end()) {                             // replace() returned "added"
        ++a;
        Au.emplace(v, Entry{W[i], b});
        if (!cand.empty()) cand.erase(key_of(u, v));
      } else if (it->second.batch != b) {               // first write of the key in this batch
        it->second = Entry{W[i], b};                    // most recent value stored
        if (!cand.empty()) cand.erase(key_of(u, v));
      } else {                                          // written before in this batch (Q1)
        auto& c = cand[key_of(u, v)];
        if (c.empty()) c.push_back(it->second.w);
        c.push_back(W[i]);
        it->second.w = W[i];
      }
    }
    added[t] = a;
  });
  uint64_t total = 0;
  for (uint64_t a : added) total += a;
  if (n_added) *n_added = total;
  return ORC_OK;
}

/* Edge deletion, §IV-C2: delete by key (u,v) (Q4); returns whether
 * the key existed, which decrements the exact count.  A key deleted
 * twice in one batch counts once (Q5).  Self-loops are never stored, so (u,u)
 * is a no-op (Q3). */
int orc_delete_edges(void* h, const uint32_t* src, const uint32_t* dst, uint64_t n,
                     uint64_t* n_removed) {
  Oracle& g = *static_cast<Oracle*>(h);
  if (n_removed) *n_removed = 0;
  if (n && (!src || !dst)) return ORC_ERR_INVALID_ARGUMENT;
  if (!in_range(g, src, n) || !in_range(g, dst, n)) return ORC_ERR_VERTEX_OUT_OF_RANGE;
  std::vector<uint32_t> S, D, W;
  expand(g, src, dst, nullptr, n, S, D, W);
  const unsigned P = threads_for(g, S.size());
  std::vector<uint64_t> removed(P, 0);
  parallel(P, [&](unsigned t) {
    uint64_t r = 0;
    for (size_t i = 0; i < S.size(); ++i) {
      const uint32_t u = S[i], v = D[i];
      if (u % P != t || u == v) continue;
      if (g.A[u].erase(v)) {
        ++r;
        auto& cand = g.cand[u % g.T];
        if (!cand.empty()) cand.erase(key_of(u, v));
      }
    }
    removed[t] = r;
  });
  uint64_t total = 0;
  for (uint64_t r : removed) total += r;
  if (n_removed) *n_removed = total;
  return ORC_OK;
}

/* edgeExist / Search_Au(v): returns <v,w> or ⊥.
 * ⊥ is reported as found=0, weight=0 (Q19).  A query never mutates, so an
 * out-of-range batch is rejected before any answer is written (Q7). */
int orc_query_edges(void* h, const uint32_t* src, const uint32_t* dst, uint64_t n,
                    uint8_t* found, uint32_t* weight) {
  Oracle& g = *static_cast<Oracle*>(h);
  if (n && (!src || !dst || !found)) return ORC_ERR_INVALID_ARGUMENT;
  if (!in_range(g, src, n) || !in_range(g, dst, n)) return ORC_ERR_VERTEX_OUT_OF_RANGE;
  const unsigned P = threads_for(g, n);
  parallel(P, [&](unsigned t) {  // read-only: any split works; contiguous ranges
    const uint64_t lo = n * t / P, hi = n * (t + 1) / P;
    for (uint64_t i = lo; i < hi; ++i) {
      const uint32_t u = src[i], v = dst[i];
      auto it = g.A[u].find(v);
      const bool f = (u != v) && it != g.A[u].end();
      found[i] = f ? 1 : 0;
      if (weight) weight[i] = f ? it->second.w : 0u;
    }
  });
  return ORC_OK;
}

/* Vertex deletion, §II-A op 3 P:L171-176 and §IV-D2: A_u is deleted
 * (count := 0, Alg2:L22) and every edge whose destination is u is removed
 * (eager, Q8).  Duplicate IDs are idempotent (Q11); the ID stays valid with an
 * empty list (Q10).  Directed and undirected modes give the same result. */
int orc_delete_vertices(void* h, const uint32_t* ids, uint64_t n) {
  Oracle& g = *static_cast<Oracle*>(h);
  if (n && !ids) return ORC_ERR_INVALID_ARGUMENT;
  if (!in_range(g, ids, n)) return ORC_ERR_VERTEX_OUT_OF_RANGE;
  const std::unordered_set<uint32_t> D(ids, ids + n);
  if (D.empty()) return ORC_OK;
  for (uint32_t u : D) g.A[u].clear();
  const unsigned P = threads_for(g, g.cap);
  parallel(P, [&](unsigned t) {
    for (uint64_t x = t; x < g.cap; x += P) {
      auto& Ax = g.A[x];
      for (auto it = Ax.begin(); it != Ax.end();) {
        if (D.count(it->first)) it = Ax.erase(it);
        else ++it;
      }
    }
    for (unsigned c = t; c < g.T; c += P) {
      auto& cand = g.cand[c];
      for (auto it = cand.begin(); it != cand.end();) {
        if (D.count((uint32_t)(it->first >> 32)) || D.count((uint32_t)it->first)) it = cand.erase(it);
        else ++it;
      }
    }
  });
  return ORC_OK;
}

/* Vertex insertion, §IV-D1 P:L509-515 and §IV-A1: the vertex
 * dictionary grows to hold the new IDs; each new vertex starts with an empty
 * adjacency list (its edges then arrive through orc_insert_edges).  Existing IDs
 * are a no-op (Q12). */
int orc_insert_vertices(void* h, const uint32_t* ids, uint64_t n) {
  Oracle& g = *static_cast<Oracle*>(h);
  if (n && !ids) return ORC_ERR_INVALID_ARGUMENT;
  uint64_t need = g.cap;
  for (uint64_t i = 0; i < n; ++i) {
    if ((uint64_t)ids[i] >= kMaxVertices) return ORC_ERR_VERTEX_OUT_OF_RANGE;
    need = std::max<uint64_t>(need, (uint64_t)ids[i] + 1);
  }
  g.cap = need;
  g.A.resize(need);
  return ORC_OK;
}

uint64_t orc_num_edges(void* h) {
  Oracle& g = *static_cast<Oracle*>(h);
  uint64_t m = 0;
  for (auto& a : g.A) m += a.size();
  return m;
}

/* Retrieve adjacency lists (§II-A op 1) for every vertex as CSR,
 * each row sorted by destination (the canonical form compared against). */
void orc_export(void* h, uint64_t* row_offsets, uint32_t* dst, uint32_t* weight) {
  Oracle& g = *static_cast<Oracle*>(h);
  uint64_t pos = 0;
  for (uint64_t u = 0; u < g.cap; ++u) {
    row_offsets[u] = pos;
    pos += g.A[u].size();
  }
  row_offsets[g.cap] = pos;
  const unsigned P = threads_for(g, pos);
  parallel(P, [&](unsigned t) {  // rows are independent: contiguous row ranges
    std::vector<std::pair<uint32_t, uint32_t>> row;
    const uint64_t lo = g.cap * t / P, hi = g.cap * (t + 1) / P;
    for (uint64_t u = lo; u < hi; ++u) {
      row.clear();
      for (auto& kv : g.A[u]) row.emplace_back(kv.first, kv.second.w);
      std::sort(row.begin(), row.end());
      uint64_t p = row_offsets[u];
      for (auto& e : row) {
        if (dst) dst[p] = e.first;
        if (weight) weight[p] = e.second;
        ++p;
      }
    }
  });
}

/* exact number of neighbours per vertex */
void orc_degrees(void* h, uint32_t* out) {
  Oracle& g = *static_cast<Oracle*>(h);
  for (uint64_t u = 0; u < g.cap; ++u) out[u] = (uint32_t)g.A[u].size();
}

/* Q1 candidate sets: writes up to `cap` triples (u, v, w); returns the total. */
uint64_t orc_candidates(void* h, uint32_t* u, uint32_t* v, uint32_t* w, uint64_t cap) {
  Oracle& g = *static_cast<Oracle*>(h);
  uint64_t k = 0;
  for (auto& shard : g.cand)
    for (auto& kv : shard)
      for (uint32_t x : kv.second) {
        if (k < cap) { u[k] = (uint32_t)(kv.first >> 32); v[k] = (uint32_t)kv.first; w[k] = x; }
        ++k;
      }
  return k;
}

/* Triangle count of the simple undirected graph held (config 5; §VI-C
 * P:L848-864).  Each triangle counted once (Q23).  This is the classic forward
 * algorithm on sorted neighbour lists — a different algorithm from the GPU's
 * per-wedge hash probes: orient each edge from lower to higher rank, rank(x) =
 * (deg x, x), and sum |N+(u) ∩ N+(v)| over oriented edges (u,v). */
uint64_t orc_triangle_count(void* h) {
  Oracle& g = *static_cast<Oracle*>(h);
  const uint64_t n = g.cap;
  auto rank_less = [&](uint32_t a, uint32_t b) {
    size_t da = g.A[a].size(), db = g.A[b].size();
    return da < db || (da == db && a < b);
  };
  std::vector<std::vector<uint32_t>> Np(n);
  parallel(g.T, [&](unsigned t) {
    for (uint64_t u = t; u < n; u += g.T) {
      for (auto& kv : g.A[u])
        if (rank_less((uint32_t)u, kv.first)) Np[u].push_back(kv.first);
      std::sort(Np[u].begin(), Np[u].end());
    }
  });
  std::vector<uint64_t> part(g.T, 0);
  parallel(g.T, [&](unsigned t) {
    uint64_t count = 0;
    for (uint64_t u = t; u < n; u += g.T)
      for (uint32_t v : Np[u]) {
        const auto& a = Np[u];
        const auto& b = Np[v];
        size_t i = 0, j = 0;
        while (i < a.size() && j < b.size()) {
          if (a[i] < b[j]) ++i;
          else if (a[i] > b[j]) ++j;
          else { ++count; ++i; ++j; }
        }
      }
    part[t] = count;
  });
  uint64_t count = 0;
  for (uint64_t c : part) count += c;
  return count;
}

/* Initial bucket count of a vertex's table, §IV-A2 P:L411-414:
 *     ceil(|A_u| / (lf * Bc)),   and a single bucket when |A_u| is unknown
 * (P:L340-342, L428-429).  lf is given in thousandths so the ceiling is an exact
 * integer decision (reading R-LF). A hint of 0 means "unknown". */
uint64_t orc_initial_buckets(uint64_t hint, uint64_t lf_milli, uint64_t bucket_capacity) {
  if (hint == 0) return 1;
  const uint64_t den = lf_milli * bucket_capacity;
  const uint64_t b = (hint * 1000 + den - 1) / den;
  return b ? b : 1;
}

}  // extern "C"
