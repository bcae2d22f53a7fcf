/*
 * synth.c -- seeded synthetic bipartite-graph generators (CSR, rows -> cols).
 *
 * This module is shared by the oracle side and the CUDA side ONLY as an input
 * source.  It contains none of the matching method's arithmetic: it draws
 * patterns, deduplicates them and emits CSR.  Every random decision comes from a
 * counter-based hash keyed by (seed, stream, index), so the output is identical
 * for any thread count.
 *
 * Recipes:
 *   uniform   : m x n, `samples` i.i.d. uniform (row, col) draws, dedup, sorted
 *               (C1: 10,000^2 x 80,000;  C5: 2^21 x 16*2^21).
 *   banded    : n x n permuted banded "circuit-like" (C2, Hamrle3-like P:918):
 *               full diagonal + Poisson(lambda) off-diagonals per row at offsets
 *               U[-w, w]\{0} (out-of-range dropped) + `rails` dense columns x
 *               `rail_len` random rows; dedup; independent random row and column
 *               permutations; sorted adjacency.
 *   road      : s x s planted-perfect road-like lattice (C3): every horizontal
 *               domino (x, x+1), x even, is kept; other horizontals w.p. a,
 *               verticals w.p. b, down-right diagonals w.p. c; symmetric pattern
 *               (row i-col j and row j-col i per kept edge), no self loops;
 *               row-major numbering, then one symmetric relabel permuting ids
 *               inside blocks of `scramble` consecutive ids (seeded); optional
 *               per-list shuffle (only visible when no relabel is applied).
 *   rmat      : 2^scale x 2^scale, `samples` R-MAT draws with (a,b,c,d) (C4,
 *               Graph500 0.57/0.19/0.19/0.05); dedup; random row and column
 *               permutations; sorted adjacency.
 *   from_pairs: build a deduplicated sorted CSR from explicit (row, col) pairs
 *               (used by the small closed-form families in synth/__init__.py).
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#include <math.h>
#include <omp.h>

typedef struct {
  int32_t m, n;
  int64_t nnz;
  int32_t *indptr;  /* m+1 */
  int32_t *indices; /* nnz */
} synth_csr_t;

/* ---------------- counter-based RNG ---------------- */
static inline uint64_t mix64(uint64_t z) {
  z += 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}
static inline uint64_t h3(uint64_t seed, uint64_t stream, uint64_t idx) {
  return mix64(mix64(seed * 0xD1B54A32D192ED03ull + stream) ^ (idx * 0x9E3779B97F4A7C15ull));
}
/* uniform integer in [0, r) by multiply-high (r < 2^32) */
static inline uint32_t below(uint64_t x, uint32_t r) { return (uint32_t)(((x >> 32) * (uint64_t)r) >> 32); }
/* uniform double in [0,1) */
static inline double unit(uint64_t x) { return (double)(x >> 11) * (1.0 / 9007199254740992.0); }

/* ---------------- helpers ---------------- */
static int cmp_i32(const void *a, const void *b) {
  int32_t x = *(const int32_t *)a, y = *(const int32_t *)b;
  return (x > y) - (x < y);
}
static void sort_small(int32_t *a, int64_t len) {
  if (len <= 24) {
    for (int64_t i = 1; i < len; i++) {
      int32_t v = a[i]; int64_t j = i - 1;
      while (j >= 0 && a[j] > v) { a[j + 1] = a[j]; j--; }
      a[j + 1] = v;
    }
  } else {
    qsort(a, (size_t)len, sizeof(int32_t), cmp_i32);
  }
}

/*
 * Bucket (row, col) pairs by row, sort + dedup each row, emit CSR.
 * rows/cols have `cnt` entries (int32).  Deterministic for any thread count
 * because each row list is sorted before dedup.
 */
static int build_csr(int32_t m, int32_t n, const int32_t *rows, const int32_t *cols, int64_t cnt,
                     int dedup, synth_csr_t *out) {
  int64_t *deg = (int64_t *)calloc((size_t)m + 1, sizeof(int64_t));
  if (!deg) return -1;
#pragma omp parallel for schedule(static)
  for (int64_t e = 0; e < cnt; e++) {
#pragma omp atomic
    deg[rows[e] + 1]++;
  }
  for (int32_t i = 0; i < m; i++) deg[i + 1] += deg[i];
  int64_t *cur = (int64_t *)malloc(sizeof(int64_t) * ((size_t)m + 1));
  int32_t *tmp = (int32_t *)malloc(sizeof(int32_t) * (size_t)(cnt > 0 ? cnt : 1));
  if (!cur || !tmp) { free(deg); free(cur); free(tmp); return -1; }
  memcpy(cur, deg, sizeof(int64_t) * ((size_t)m + 1));
#pragma omp parallel for schedule(static)
  for (int64_t e = 0; e < cnt; e++) {
    int64_t p;
#pragma omp atomic capture
    p = cur[rows[e]]++;
    tmp[p] = cols[e];
  }
  /* sort + dedup per row; new lengths into cur[i] */
#pragma omp parallel for schedule(dynamic, 1024)
  for (int32_t i = 0; i < m; i++) {
    int32_t *a = tmp + deg[i];
    int64_t len = deg[i + 1] - deg[i];
    sort_small(a, len);
    int64_t k = 0;
    for (int64_t j = 0; j < len; j++)
      if (!dedup || k == 0 || a[j] != a[k - 1]) a[k++] = a[j];
    cur[i] = k;
  }
  out->m = m; out->n = n;
  out->indptr = (int32_t *)malloc(sizeof(int32_t) * ((size_t)m + 1));
  int64_t tot = 0;
  for (int32_t i = 0; i < m; i++) tot += cur[i];
  out->nnz = tot;
  out->indices = (int32_t *)malloc(sizeof(int32_t) * (size_t)(tot > 0 ? tot : 1));
  if (!out->indptr || !out->indices || tot >= ((int64_t)1 << 31)) { free(deg); free(cur); free(tmp); return -1; }
  int64_t *off = (int64_t *)malloc(sizeof(int64_t) * ((size_t)m + 1));
  off[0] = 0;
  for (int32_t i = 0; i < m; i++) off[i + 1] = off[i] + cur[i];
#pragma omp parallel for schedule(static)
  for (int32_t i = 0; i < m; i++) {
    out->indptr[i] = (int32_t)off[i];
    memcpy(out->indices + off[i], tmp + deg[i], sizeof(int32_t) * (size_t)cur[i]);
  }
  out->indptr[m] = (int32_t)off[m];
  free(off); free(deg); free(cur); free(tmp);
  return 0;
}

/* seeded Fisher-Yates permutation of 0..len-1 (sequential splitmix stream) */
static int32_t *make_perm(int32_t len, uint64_t seed, uint64_t stream) {
  int32_t *p = (int32_t *)malloc(sizeof(int32_t) * (size_t)(len > 0 ? len : 1));
  if (!p) return NULL;
  for (int32_t i = 0; i < len; i++) p[i] = i;
  for (int64_t i = (int64_t)len - 1; i > 0; i--) {
    uint64_t x = h3(seed, stream, (uint64_t)i);
    int32_t j = (int32_t)below(x, (uint32_t)(i + 1));
    int32_t t = p[i]; p[i] = p[j]; p[j] = t;
  }
  return p;
}

void synth_free(synth_csr_t *g) {
  if (!g) return;
  free(g->indptr); free(g->indices);
  g->indptr = NULL; g->indices = NULL;
}

int synth_set_threads(int t) { if (t > 0) omp_set_num_threads(t); return omp_get_max_threads(); }

/* ---------------- families ---------------- */

int synth_from_pairs(int32_t m, int32_t n, const int32_t *rows, const int32_t *cols, int64_t cnt,
                     synth_csr_t *out) {
  for (int64_t e = 0; e < cnt; e++)
    if (rows[e] < 0 || rows[e] >= m || cols[e] < 0 || cols[e] >= n) return -2;
  return build_csr(m, n, rows, cols, cnt, 1, out);
}

int synth_uniform(int32_t m, int32_t n, int64_t samples, uint64_t seed, synth_csr_t *out) {
  if (m <= 0 || n <= 0) { samples = 0; }
  int32_t *r = (int32_t *)malloc(sizeof(int32_t) * (size_t)(samples > 0 ? samples : 1));
  int32_t *c = (int32_t *)malloc(sizeof(int32_t) * (size_t)(samples > 0 ? samples : 1));
  if (!r || !c) return -1;
#pragma omp parallel for schedule(static)
  for (int64_t e = 0; e < samples; e++) {
    r[e] = (int32_t)below(h3(seed, 1, (uint64_t)e), (uint32_t)m);
    c[e] = (int32_t)below(h3(seed, 2, (uint64_t)e), (uint32_t)n);
  }
  int rc = build_csr(m, n, r, c, samples, 1, out);
  free(r); free(c);
  return rc;
}

/* Poisson(lambda) by inverse CDF from one uniform (lambda small) */
static int poisson_icdf(double lambda, double u) {
  double p = exp(-lambda), s = p;
  int k = 0;
  while (u > s && k < 64) { k++; p *= lambda / k; s += p; }
  return k;
}

int synth_banded(int32_t n, double lambda, int32_t w, int32_t rails, int32_t rail_len, uint64_t seed,
                 int permute, synth_csr_t *out) {
  /* per-row count of off-diagonals */
  int32_t *k = (int32_t *)malloc(sizeof(int32_t) * (size_t)n);
  int64_t *off = (int64_t *)malloc(sizeof(int64_t) * ((size_t)n + 1));
  if (!k || !off) return -1;
#pragma omp parallel for schedule(static)
  for (int32_t i = 0; i < n; i++) k[i] = poisson_icdf(lambda, unit(h3(seed, 3, (uint64_t)i)));
  off[0] = 0;
  for (int32_t i = 0; i < n; i++) off[i + 1] = off[i] + 1 + k[i];
  int64_t total = off[n] + (int64_t)rails * rail_len;
  int32_t *r = (int32_t *)malloc(sizeof(int32_t) * (size_t)total);
  int32_t *c = (int32_t *)malloc(sizeof(int32_t) * (size_t)total);
  if (!r || !c) return -1;
  int64_t keep_bad = 0;
#pragma omp parallel for schedule(static) reduction(+ : keep_bad)
  for (int32_t i = 0; i < n; i++) {
    int64_t p = off[i];
    r[p] = i; c[p] = i; p++;
    for (int32_t j = 0; j < k[i]; j++, p++) {
      int32_t d = (int32_t)below(h3(seed, 4, (uint64_t)i * 64 + j), (uint32_t)(2 * w)) - w;
      if (d >= 0) d++; /* U[-w,w] \ {0} */
      int64_t col = (int64_t)i + d;
      if (col < 0 || col >= n) { col = i; keep_bad++; } /* dropped: duplicate of diagonal, removed by dedup */
      r[p] = i; c[p] = (int32_t)col;
    }
  }
  for (int32_t q = 0; q < rails; q++) {
    int32_t col = (int32_t)below(h3(seed, 5, (uint64_t)q), (uint32_t)n);
    for (int32_t t = 0; t < rail_len; t++) {
      int64_t p = off[n] + (int64_t)q * rail_len + t;
      r[p] = (int32_t)below(h3(seed, 6, (uint64_t)p), (uint32_t)n);
      c[p] = col;
    }
  }
  if (permute) {
    int32_t *pr = make_perm(n, seed, 7), *pc = make_perm(n, seed, 8);
#pragma omp parallel for schedule(static)
    for (int64_t e = 0; e < total; e++) { r[e] = pr[r[e]]; c[e] = pc[c[e]]; }
    free(pr); free(pc);
  }
  int rc = build_csr(n, n, r, c, total, 1, out);
  free(k); free(off); free(r); free(c);
  return rc;
}

/* road lattice: vertex id = y*s + x */
static inline int keep_h(uint64_t seed, int32_t s, int32_t x, int32_t y, double a) {
  if (x < 0 || x + 1 >= s || y < 0 || y >= s) return 0;
  if ((x & 1) == 0) return 1; /* planted domino */
  return unit(h3(seed, 10, (uint64_t)y * s + x)) < a;
}
static inline int keep_v(uint64_t seed, int32_t s, int32_t x, int32_t y, double b) {
  if (x < 0 || x >= s || y < 0 || y + 1 >= s) return 0;
  return unit(h3(seed, 11, (uint64_t)y * s + x)) < b;
}
static inline int keep_d(uint64_t seed, int32_t s, int32_t x, int32_t y, double c) {
  if (x < 0 || x + 1 >= s || y < 0 || y + 1 >= s) return 0;
  return unit(h3(seed, 12, (uint64_t)y * s + x)) < c;
}
static int road_nbrs(uint64_t seed, int32_t s, int32_t x, int32_t y, double a, double b, double c,
                     int32_t *nb) {
  int k = 0;
  if (keep_h(seed, s, x, y, a)) nb[k++] = y * s + x + 1;          /* right */
  if (keep_h(seed, s, x - 1, y, a)) nb[k++] = y * s + x - 1;      /* left */
  if (keep_v(seed, s, x, y, b)) nb[k++] = (y + 1) * s + x;        /* down */
  if (keep_v(seed, s, x, y - 1, b)) nb[k++] = (y - 1) * s + x;    /* up */
  if (keep_d(seed, s, x, y, c)) nb[k++] = (y + 1) * s + x + 1;    /* down-right */
  if (keep_d(seed, s, x - 1, y - 1, c)) nb[k++] = (y - 1) * s + x - 1; /* up-left */
  return k;
}

int synth_road(int32_t s, double a, double b, double c, uint64_t seed, int shuffle, int permute,
               int32_t scramble, synth_csr_t *out) {
  int64_t N = (int64_t)s * s;
  if (N >= ((int64_t)1 << 31) - 2) return -2;
  int32_t *deg = (int32_t *)malloc(sizeof(int32_t) * (size_t)(N > 0 ? N : 1));
  int64_t *off = (int64_t *)malloc(sizeof(int64_t) * ((size_t)N + 1));
  if (!deg || !off) return -1;
#pragma omp parallel for schedule(static)
  for (int64_t v = 0; v < N; v++) {
    int32_t nb[8];
    deg[v] = road_nbrs(seed, s, (int32_t)(v % s), (int32_t)(v / s), a, b, c, nb);
  }
  off[0] = 0;
  for (int64_t v = 0; v < N; v++) off[v + 1] = off[v] + deg[v];
  if (off[N] >= ((int64_t)1 << 31)) return -2;
  int32_t *adj = (int32_t *)malloc(sizeof(int32_t) * (size_t)(off[N] > 0 ? off[N] : 1));
  if (!adj) return -1;
#pragma omp parallel for schedule(static)
  for (int64_t v = 0; v < N; v++) {
    int32_t nb[8];
    int k = road_nbrs(seed, s, (int32_t)(v % s), (int32_t)(v / s), a, b, c, nb);
    if (shuffle)
      for (int i = k - 1; i > 0; i--) {
        int j = (int)below(h3(seed, 13, (uint64_t)v * 8 + i), (uint32_t)(i + 1));
        int32_t t = nb[i]; nb[i] = nb[j]; nb[j] = t;
      }
    memcpy(adj + off[v], nb, sizeof(int32_t) * k);
  }
  if (permute || scramble > 1) {
    /* permute: relabel rows and columns independently (C3-perm);
     * scramble: one symmetric relabel that permutes ids inside consecutive
     * blocks of `scramble` ids (locality kept at block granularity, but the
     * id order no longer favours the planted dominoes).  Rebuild sorted CSR. */
    int32_t *pr, *pc;
    if (permute) { pr = make_perm((int32_t)N, seed, 14); pc = make_perm((int32_t)N, seed, 15); }
    else {
      pr = (int32_t *)malloc(sizeof(int32_t) * (size_t)N);
#pragma omp parallel for schedule(static)
      for (int64_t b0 = 0; b0 < N; b0 += scramble) {
        int64_t len = (N - b0 < scramble) ? N - b0 : scramble;
        for (int64_t i = 0; i < len; i++) pr[b0 + i] = (int32_t)(b0 + i);
        for (int64_t i = len - 1; i > 0; i--) {
          int64_t j = below(h3(seed, 16, (uint64_t)(b0 + i)), (uint32_t)(i + 1));
          int32_t t = pr[b0 + i]; pr[b0 + i] = pr[b0 + j]; pr[b0 + j] = t;
        }
      }
      pc = pr;
    }
    int32_t *r = (int32_t *)malloc(sizeof(int32_t) * (size_t)off[N]);
#pragma omp parallel for schedule(static)
    for (int64_t v = 0; v < N; v++)
      for (int64_t e = off[v]; e < off[v + 1]; e++) { r[e] = pr[v]; adj[e] = pc[adj[e]]; }
    int rc = build_csr((int32_t)N, (int32_t)N, r, adj, off[N], 1, out);
    if (pc != pr) free(pc);
    free(pr); free(r); free(adj); free(deg); free(off);
    return rc;
  }
  out->m = (int32_t)N; out->n = (int32_t)N; out->nnz = off[N];
  out->indptr = (int32_t *)malloc(sizeof(int32_t) * ((size_t)N + 1));
#pragma omp parallel for schedule(static)
  for (int64_t v = 0; v <= N; v++) out->indptr[v] = (int32_t)off[v];
  out->indices = adj;
  free(deg); free(off);
  return 0;
}

int synth_rmat(int32_t scale, int64_t samples, double a, double b, double c, uint64_t seed, int permute,
               synth_csr_t *out) {
  if (scale < 1 || scale > 30) return -2;
  int32_t N = (int32_t)1 << scale;
  int32_t *r = (int32_t *)malloc(sizeof(int32_t) * (size_t)(samples > 0 ? samples : 1));
  int32_t *cc = (int32_t *)malloc(sizeof(int32_t) * (size_t)(samples > 0 ? samples : 1));
  if (!r || !cc) return -1;
  const double ab = a + b, abc = a + b + c;
#pragma omp parallel for schedule(static)
  for (int64_t e = 0; e < samples; e++) {
    uint32_t row = 0, col = 0;
    for (int32_t l = 0; l < scale; l++) {
      double u = unit(h3(seed, 20 + (uint64_t)l, (uint64_t)e));
      int q = u < a ? 0 : (u < ab ? 1 : (u < abc ? 2 : 3));
      row = (row << 1) | (uint32_t)(q >> 1);
      col = (col << 1) | (uint32_t)(q & 1);
    }
    r[e] = (int32_t)row; cc[e] = (int32_t)col;
  }
  if (permute) {
    int32_t *pr = make_perm(N, seed, 60), *pc = make_perm(N, seed, 61);
#pragma omp parallel for schedule(static)
    for (int64_t e = 0; e < samples; e++) { r[e] = pr[r[e]]; cc[e] = pc[cc[e]]; }
    free(pr); free(pc);
  }
  int rc = build_csr(N, N, r, cc, samples, 1, out);
  free(r); free(cc);
  return rc;
}
