/*
 * workloads/gen.c — seeded synthetic input generators shared by the oracle harness
 * and the GPU path.  This file holds NO arithmetic of the method (no hashing of
 * keys into buckets, no table logic): it only draws random numbers and shapes
 * them into edge lists with the structure of the paper's workloads
 * (§V-A1 P:L609-615 "randomly generated edges between existing
 * vertices"; Tab. I P:L676-690 dataset shapes; SURVEY.md §8(d) generator spec).
 *
 * Every random number comes from a counter-based generator
 *     rng(seed, stream, index) = splitmix64(splitmix64(seed ^ splitmix64(stream)) + index)
 * so any slice of any batch can be regenerated independently (a rank can produce
 * its 1/P of a batch; the oracle harness produces the whole batch bit-identically),
 * and results do not depend on the number of OpenMP threads.
 */
#include <stdint.h>
#include <stddef.h>
#include <string.h>
#include <stdlib.h>

static inline uint64_t splitmix64(uint64_t x) {
  x += 0x9E3779B97F4A7C15ULL;
  x = (x ^ (x >> 30)) * 0xBF58476D1CE4E5B9ULL;
  x = (x ^ (x >> 27)) * 0x94D049BB133111EBULL;
  return x ^ (x >> 31);
}

static inline uint64_t stream_key(uint64_t seed, uint64_t stream) {
  return splitmix64(seed ^ splitmix64(stream));
}

static inline uint64_t rng_k(uint64_t key, uint64_t index) { return splitmix64(key + index); }

/* multiply-shift range reduction of a 32-bit draw onto [0, n) */
static inline uint32_t below(uint32_t r, uint64_t n) { return (uint32_t)(((uint64_t)r * n) >> 32); }

uint64_t wl_rng(uint64_t seed, uint64_t stream, uint64_t index) {
  return rng_k(stream_key(seed, stream), index);
}

/* ---------------------------------------------------------------- uniform ---- */
/* n edges with src,dst uniform on [0, nv) (self-loops and duplicates occur
 * naturally), weights uniform u32.  w may be NULL. */
void wl_uniform_edges(uint64_t seed, uint64_t stream, uint64_t i0, uint64_t n, uint64_t nv,
                      uint32_t* src, uint32_t* dst, uint32_t* w) {
  const uint64_t k = stream_key(seed, stream);
  const uint64_t kw = stream_key(seed, stream ^ 0x5757575757575757ULL);
#pragma omp parallel for schedule(static)
  for (int64_t i = 0; i < (int64_t)n; ++i) {
    uint64_t r = rng_k(k, i0 + (uint64_t)i);
    src[i] = below((uint32_t)(r >> 32), nv);
    dst[i] = below((uint32_t)r, nv);
    if (w) w[i] = (uint32_t)(rng_k(kw, i0 + (uint64_t)i) >> 32);
  }
}

/* uniform u32 values (weights, or indices after reduction by the caller) */
void wl_uniform_u32(uint64_t seed, uint64_t stream, uint64_t i0, uint64_t n, uint64_t bound,
                    uint32_t* out) {
  const uint64_t k = stream_key(seed, stream);
#pragma omp parallel for schedule(static)
  for (int64_t i = 0; i < (int64_t)n; ++i) {
    uint32_t r = (uint32_t)(rng_k(k, i0 + (uint64_t)i) >> 32);
    out[i] = bound ? below(r, bound) : r;
  }
}

/* uniform u64 indices on [0, bound) (for sampling from long edge lists) */
void wl_uniform_index(uint64_t seed, uint64_t stream, uint64_t n, uint64_t bound, uint64_t* out) {
  const uint64_t k = stream_key(seed, stream);
#pragma omp parallel for schedule(static)
  for (int64_t i = 0; i < (int64_t)n; ++i) {
    out[i] = rng_k(k, (uint64_t)i) % (bound ? bound : 1);
  }
}

/* --------------------------------------------------------- ID permutation ---- */
/* A 4-round balanced Feistel bijection on [0, 2^(2h)) with cycle walking into
 * [0, 2^scale), h = ceil(scale/2).  Keyed by the seed; no stored permutation. */
static inline uint32_t feistel_once(uint32_t x, int h, uint64_t key) {
  const uint32_t mask = (h >= 32) ? 0xFFFFFFFFu : ((1u << h) - 1u);
  uint32_t L = (x >> h) & mask, R = x & mask;
  for (int r = 0; r < 4; ++r) {
    uint32_t F = (uint32_t)splitmix64(key + (uint64_t)r * 0x100000001ULL + R) & mask;
    uint32_t nL = R, nR = L ^ F;
    L = nL; R = nR;
  }
  return (L << h) | R;
}

uint32_t wl_permute(uint32_t x, int scale, uint64_t seed) {
  const int h = (scale + 1) / 2;
  const uint64_t key = splitmix64(seed ^ 0xFE15FE15FE15FE15ULL);
  const uint64_t lim = 1ULL << scale;
  uint32_t y = feistel_once(x, h, key);
  while ((uint64_t)y >= lim) y = feistel_once(y, h, key);
  return y;
}

/* ------------------------------------------------------------------ R-MAT ---- */
/* Edge i, level l: one uniform decides the quadrant with probabilities
 * (a, b, c, 1-a-b-c), no noise.  IDs optionally permuted (Feistel above).
 * nv < 2^scale: attempt j = 0,1,... of edge i is retried until both endpoints
 * are < nv (deterministic rejection, SURVEY §8(d) "LJ-like rejection"). */
static inline void rmat_one(uint64_t key, uint64_t i, uint64_t attempt, int scale,
                            uint32_t ta, uint32_t tab, uint32_t tabc,
                            uint32_t* s, uint32_t* d) {
  uint32_t u = 0, v = 0;
  const uint64_t base = (i * 64ULL) ^ (attempt << 56);
  for (int l = 0; l < scale; ++l) {
    uint32_t r = (uint32_t)(rng_k(key, base + (uint64_t)l) >> 32);
    uint32_t bu, bv;
    if (r < ta) { bu = 0; bv = 0; }
    else if (r < tab) { bu = 0; bv = 1; }
    else if (r < tabc) { bu = 1; bv = 0; }
    else { bu = 1; bv = 1; }
    u = (u << 1) | bu;
    v = (v << 1) | bv;
  }
  *s = u; *d = v;
}

/* edge ids: idx[i] if idx != NULL, else i0 + i */
void wl_rmat_edges(uint64_t seed, uint64_t stream, uint64_t i0, const uint64_t* idx, uint64_t n,
                   int scale, double a, double b, double c, int permute, uint64_t nv,
                   uint32_t* src, uint32_t* dst) {
  const uint64_t key = stream_key(seed, stream);
  const double two32 = 4294967296.0;
  double fa = a * two32, fab = (a + b) * two32, fabc = (a + b + c) * two32;
  uint32_t ta = fa >= two32 ? 0xFFFFFFFFu : (uint32_t)fa;
  uint32_t tab = fab >= two32 ? 0xFFFFFFFFu : (uint32_t)fab;
  uint32_t tabc = fabc >= two32 ? 0xFFFFFFFFu : (uint32_t)fabc;
  const uint64_t full = 1ULL << scale;
  if (nv == 0 || nv > full) nv = full;
#pragma omp parallel for schedule(static)
  for (int64_t i = 0; i < (int64_t)n; ++i) {
    uint32_t s, d;
    const uint64_t e = idx ? idx[i] : i0 + (uint64_t)i;
    for (uint64_t att = 0;; ++att) {
      rmat_one(key, e, att, scale, ta, tab, tabc, &s, &d);
      if (permute) { s = wl_permute(s, scale, seed); d = wl_permute(d, scale, seed); }
      if (s < nv && d < nv) break;
    }
    src[i] = s; dst[i] = d;
  }
}

/* ---------------------------------------------------------- road-like grid ---- */
/* rows x cols lattice, vertex id = r*cols + c.  Each undirected lattice edge is
 * kept with probability p (keep iff rng < p*2^64); both directions are emitted.
 * Pass src==NULL to get the count only.  Output is in row-major vertex order. */
static inline int keep_edge(uint64_t key, uint64_t idx, uint64_t thr) { return rng_k(key, idx) < thr; }
#define KEEP(i) (keep_edge(key, (i), thr) != held_out)

static uint64_t grid_edges(uint64_t seed, uint64_t rows, uint64_t cols, double p, int held_out,
                           uint32_t* src, uint32_t* dst);

uint64_t wl_grid_edges(uint64_t seed, uint64_t rows, uint64_t cols, double p,
                       uint32_t* src, uint32_t* dst) {
  return grid_edges(seed, rows, cols, p, 0, src, dst);
}

/* the lattice edges the grid did NOT keep (road-network growth workload, SURVEY
 * §8(d) cfg3 "held-out lattice edges"), both directions, same order */
uint64_t wl_grid_heldout_edges(uint64_t seed, uint64_t rows, uint64_t cols, double p,
                               uint32_t* src, uint32_t* dst) {
  return grid_edges(seed, rows, cols, p, 1, src, dst);
}

static uint64_t grid_edges(uint64_t seed, uint64_t rows, uint64_t cols, double p, int held_out,
                           uint32_t* src, uint32_t* dst) {
  const uint64_t key = stream_key(seed, 0x67726964ULL);
  const double two64 = 18446744073709551616.0;
  const uint64_t thr = p >= 1.0 ? 0xFFFFFFFFFFFFFFFFULL : (uint64_t)(p * two64);
  const uint64_t nv = rows * cols;
  /* per-row directed-edge counts, then prefix, then fill (deterministic order) */
  uint64_t* rowcnt = (uint64_t*)calloc(rows + 1, sizeof(uint64_t));
#pragma omp parallel for schedule(static)
  for (int64_t r = 0; r < (int64_t)rows; ++r) {
    uint64_t cnt = 0;
    for (uint64_t c = 0; c < cols; ++c) {
      uint64_t id = (uint64_t)r * cols + c;
      /* out-edges of id: right, left, down, up */
      if (c + 1 < cols && KEEP(2 * id)) cnt++;
      if (c > 0 && KEEP(2 * (id - 1))) cnt++;
      if ((uint64_t)r + 1 < rows && KEEP(2 * id + 1)) cnt++;
      if (r > 0 && KEEP(2 * (id - cols) + 1)) cnt++;
    }
    rowcnt[r + 1] = cnt;
  }
  for (uint64_t r = 0; r < rows; ++r) rowcnt[r + 1] += rowcnt[r];
  uint64_t total = rowcnt[rows];
  if (src && dst) {
#pragma omp parallel for schedule(static)
    for (int64_t r = 0; r < (int64_t)rows; ++r) {
      uint64_t pos = rowcnt[r];
      for (uint64_t c = 0; c < cols; ++c) {
        uint64_t id = (uint64_t)r * cols + c;
        if (c + 1 < cols && KEEP(2 * id)) { src[pos] = (uint32_t)id; dst[pos] = (uint32_t)(id + 1); pos++; }
        if (c > 0 && KEEP(2 * (id - 1))) { src[pos] = (uint32_t)id; dst[pos] = (uint32_t)(id - 1); pos++; }
        if ((uint64_t)r + 1 < rows && KEEP(2 * id + 1)) { src[pos] = (uint32_t)id; dst[pos] = (uint32_t)(id + cols); pos++; }
        if (r > 0 && KEEP(2 * (id - cols) + 1)) { src[pos] = (uint32_t)id; dst[pos] = (uint32_t)(id - cols); pos++; }
      }
    }
  }
  (void)nv;
  free(rowcnt);
  return total;
}

/* out-degree histogram of an edge list (input shaping only: hints for dg_create
 * are "connectivity information" the user already has). */
void wl_out_degrees(const uint32_t* src, uint64_t n, uint64_t nv, uint32_t* deg) {
  memset(deg, 0, nv * sizeof(uint32_t));
  for (uint64_t i = 0; i < n; ++i) deg[src[i]]++;
}
