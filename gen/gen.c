/*
 * gen.c -- seeded synthetic input generators shared by the oracle tests and
 * the CUDA path.  This module holds NONE of the method's arithmetic (no SpMV,
 * no CG): it only builds CSR matrices and vectors with the shapes, sizes and
 * structure of the paper's workloads (DESIGN.md section 4 states the recipe).
 *
 *   gen_makea   : NAS CG "makea" [ext:NPB] -- the matrix of the NAS CG
 *                 benchmark whose SpMV the paper maps to cuSPARSE (Fig. 4,
 *                 P:345-349).  Reproduced from the NPB
 *                 definition: randlc LCG (a=5^13, mod 2^46, seed 314159265,
 *                 one draw discarded), sprnvc/vecset outer vectors, sparse()
 *                 summing the outer products in generation order.
 *   gen_powerlaw: Parboil-spmv-shaped power-law rows (BJ.cfg[2]; the paper's
 *                 Parboil format is not named, reading R18).
 *   gen_stencil27: 27-point Laplacian, Dirichlet truncation (BJ.cfg[4], R19).
 *   gen_uniform : U[-1,1) values from a counter-based splitmix64.
 *
 * Every generator is deterministic and single-threaded.
 */
#include <math.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

typedef struct {
    int64_t m, n, nnz;
    int32_t *rowptr;
    int32_t *colidx;
    double *vals;
} gen_csr;

void gen_free(gen_csr *g)
{
    if (!g) return;
    free(g->rowptr);
    free(g->colidx);
    free(g->vals);
    free(g);
}

int64_t gen_m(const gen_csr *g) { return g->m; }
int64_t gen_n(const gen_csr *g) { return g->n; }
int64_t gen_nnz(const gen_csr *g) { return g->nnz; }

/* copies out; vals as float64 (f32 == 0) or rounded to float32 (f32 != 0) */
void gen_copy(const gen_csr *g, int32_t *rowptr, int32_t *colidx, void *vals, int f32)
{
    memcpy(rowptr, g->rowptr, sizeof(int32_t) * (size_t)(g->m + 1));
    memcpy(colidx, g->colidx, sizeof(int32_t) * (size_t)g->nnz);
    if (!f32) {
        memcpy(vals, g->vals, sizeof(double) * (size_t)g->nnz);
    } else {
        float *v = (float *)vals;
        for (int64_t k = 0; k < g->nnz; k++) v[k] = (float)g->vals[k];
    }
}

/* ----------------------------------------------------------------------- */
/* NPB randlc: x <- a*x mod 2^46, returns x * 2^-46.  Exact in integers.   */
static const uint64_t MOD46 = (1ULL << 46) - 1;

static double randlc(uint64_t *x, uint64_t a)
{
    unsigned __int128 p = (unsigned __int128)a * (unsigned __int128)(*x);
    *x = (uint64_t)(p & MOD46);
    return (double)(*x) * 0x1.0p-46;
}

/* exposes the raw stream for pinning against a big-integer reference */
void gen_randlc_stream(uint64_t seed, uint64_t a, int64_t count, double *out)
{
    uint64_t x = seed;
    for (int64_t i = 0; i < count; i++) out[i] = randlc(&x, a);
}

typedef struct { int32_t col; uint32_t seq; double v; } trip;

static int trip_cmp(const void *pa, const void *pb)
{
    const trip *a = (const trip *)pa, *b = (const trip *)pb;
    if (a->col != b->col) return a->col < b->col ? -1 : 1;
    if (a->seq != b->seq) return a->seq < b->seq ? -1 : 1;
    return 0;
}

/* NAS CG makea for one class: n=NA, nonzer=NONZER, shift=SHIFT, rcond=RCOND.
 * Returns NULL on allocation failure.                                      */
gen_csr *gen_makea(int64_t n, int32_t nonzer, double rcond, double shift)
{
    const uint64_t amult = 1220703125ULL;
    uint64_t tran = 314159265ULL;
    (void)randlc(&tran, amult); /* main(): zeta = randlc(&tran, amult) */

    int64_t nn1 = 1;
    do { nn1 = 2 * nn1; } while (nn1 < n);

    if (nonzer < 1 || nonzer > 62 || n < 1) return NULL;
    int32_t w = nonzer + 1;
    int32_t *arow = malloc(sizeof(int32_t) * (size_t)n);
    int32_t *acol = malloc(sizeof(int32_t) * (size_t)n * (size_t)w);
    double *aelt = malloc(sizeof(double) * (size_t)n * (size_t)w);
    if (!arow || !acol || !aelt) { free(arow); free(acol); free(aelt); return NULL; }

    /* makea: outer vectors.  sprnvc draws (value, location) pairs, rejecting
     * locations > n and repeats; vecset puts 0.5 at position iouter+1.     */
    for (int64_t iouter = 0; iouter < n; iouter++) {
        double vc[64];
        int32_t ivc[64];
        int32_t nzv = 0;
        while (nzv < nonzer) {
            double vecelt = randlc(&tran, amult);
            double vecloc = randlc(&tran, amult);
            int64_t i = (int64_t)((double)nn1 * vecloc) + 1;
            if (i > n) continue;
            int was_gen = 0;
            for (int32_t ii = 0; ii < nzv; ii++)
                if (ivc[ii] == i) { was_gen = 1; break; }
            if (was_gen) continue;
            vc[nzv] = vecelt;
            ivc[nzv] = (int32_t)i;
            nzv++;
        }
        int set = 0;
        for (int32_t k = 0; k < nzv; k++)
            if (ivc[k] == iouter + 1) { vc[k] = 0.5; set = 1; }
        if (!set) { vc[nzv] = 0.5; ivc[nzv] = (int32_t)(iouter + 1); nzv++; }
        arow[iouter] = nzv;
        for (int32_t e = 0; e < nzv; e++) {
            acol[iouter * w + e] = ivc[e] - 1;
            aelt[iouter * w + e] = vc[e];
        }
    }

    /* sparse(): triplet (j, jcol, va) for every pair of entries of each outer
     * vector i, va = aelt[nzrow] * (size * aelt[nza]), diagonal of vector i
     * gets va + rcond - shift, size *= rcond^(1/n) per outer vector.       */
    int64_t *cnt = calloc((size_t)n + 1, sizeof(int64_t));
    if (!cnt) { free(arow); free(acol); free(aelt); return NULL; }
    int64_t ntrip = 0;
    for (int64_t i = 0; i < n; i++)
        for (int32_t nza = 0; nza < arow[i]; nza++) {
            cnt[acol[i * w + nza] + 1] += arow[i];
            ntrip += arow[i];
        }
    for (int64_t j = 0; j < n; j++) cnt[j + 1] += cnt[j];
    trip *t = malloc(sizeof(trip) * (size_t)(ntrip > 0 ? ntrip : 1));
    int64_t *fill = malloc(sizeof(int64_t) * (size_t)(n + 1));
    if (!t || !fill) { free(t); free(fill); free(cnt); free(arow); free(acol); free(aelt); return NULL; }
    memcpy(fill, cnt, sizeof(int64_t) * (size_t)(n + 1));
    double size = 1.0;
    double ratio = pow(rcond, (1.0 / (double)n));
    for (int64_t i = 0; i < n; i++) {
        for (int32_t nza = 0; nza < arow[i]; nza++) {
            int32_t j = acol[i * w + nza];
            double scale = size * aelt[i * w + nza];
            for (int32_t nzrow = 0; nzrow < arow[i]; nzrow++) {
                int32_t jcol = acol[i * w + nzrow];
                double va = aelt[i * w + nzrow] * scale;
                if (jcol == j && j == i) va = va + rcond - shift;
                trip *e = &t[fill[j]];
                e->col = jcol; e->seq = (uint32_t)(fill[j] - cnt[j]); e->v = va;
                fill[j]++;
            }
        }
        size = size * ratio;
    }
    /* per row: order by column (stable in generation order), then sum the
     * duplicates in generation order starting from 0.0 (a[k] = a[k] + va). */
    int64_t nnz = 0;
    for (int64_t j = 0; j < n; j++) {
        qsort(t + cnt[j], (size_t)(cnt[j + 1] - cnt[j]), sizeof(trip), trip_cmp);
        int64_t k = cnt[j];
        while (k < cnt[j + 1]) { int32_t c = t[k].col; while (k < cnt[j + 1] && t[k].col == c) k++; nnz++; }
    }
    gen_csr *g = calloc(1, sizeof(gen_csr));
    g->m = n; g->n = n; g->nnz = nnz;
    g->rowptr = malloc(sizeof(int32_t) * (size_t)(n + 1));
    g->colidx = malloc(sizeof(int32_t) * (size_t)(nnz > 0 ? nnz : 1));
    g->vals = malloc(sizeof(double) * (size_t)(nnz > 0 ? nnz : 1));
    if (!g->rowptr || !g->colidx || !g->vals) { gen_free(g); g = NULL; goto out; }
    int64_t o = 0;
    g->rowptr[0] = 0;
    for (int64_t j = 0; j < n; j++) {
        int64_t k = cnt[j];
        while (k < cnt[j + 1]) {
            int32_t c = t[k].col;
            double a = 0.0;
            while (k < cnt[j + 1] && t[k].col == c) { a = a + t[k].v; k++; }
            g->colidx[o] = c; g->vals[o] = a; o++;
        }
        g->rowptr[j + 1] = (int32_t)o;
    }
out:
    free(t); free(fill); free(cnt); free(arow); free(acol); free(aelt);
    return g;
}

/* ----------------------------------------------------------------------- */
/* counter-based splitmix64: value = mix(mix(seed ^ stream<<56) + counter) */
static uint64_t mix64(uint64_t z)
{
    z += 0x9E3779B97F4A7C15ULL;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ULL;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBULL;
    return z ^ (z >> 31);
}

static uint64_t rng(uint64_t seed, uint64_t stream, uint64_t ctr)
{
    return mix64(mix64(seed ^ (stream << 56)) + ctr);
}

/* U[-1,1) with 53 random bits (exact in double, and rounded once to float) */
static double u11(uint64_t seed, uint64_t stream, uint64_t ctr)
{
    return (double)(rng(seed, stream, ctr) >> 11) * 0x1.0p-52 - 1.0;
}

void gen_uniform_f64(uint64_t seed, uint64_t stream, int64_t count, double *out)
{
    for (int64_t i = 0; i < count; i++) out[i] = u11(seed, stream, (uint64_t)i);
}

void gen_uniform_f32(uint64_t seed, uint64_t stream, int64_t count, float *out)
{
    for (int64_t i = 0; i < count; i++) out[i] = (float)u11(seed, stream, (uint64_t)i);
}

int cmp_i32(const void *a, const void *b)
{
    int32_t x = *(const int32_t *)a, y = *(const int32_t *)b;
    return (x > y) - (x < y);
}

/* Parboil-shaped power-law CSR (BJ.cfg[2]):
 *   row length by rank r=1..m: L(r) = max(1, floor(lmax * r^-beta)), capped at n;
 *   ranks assigned to rows by a seeded Fisher-Yates permutation (stream 1);
 *   columns: L distinct uniform in [0,n) by Floyd's algorithm (stream 2),
 *   sorted ascending; values U[-1,1) (stream 3, counter = nnz index).       */
gen_csr *gen_powerlaw(int64_t m, int64_t n, double lmax, double beta, uint64_t seed)
{
    int32_t *len = malloc(sizeof(int32_t) * (size_t)(m > 0 ? m : 1));
    int64_t *perm = malloc(sizeof(int64_t) * (size_t)(m > 0 ? m : 1));
    if (!len || !perm) { free(len); free(perm); return NULL; }
    for (int64_t i = 0; i < m; i++) perm[i] = i;
    for (int64_t i = m - 1; i > 0; i--) {
        uint64_t r = rng(seed, 1, (uint64_t)i);
        int64_t j = (int64_t)(((unsigned __int128)r * (unsigned __int128)(i + 1)) >> 64);
        int64_t tmp = perm[i]; perm[i] = perm[j]; perm[j] = tmp;
    }
    for (int64_t r = 1; r <= m; r++) {
        double l = floor(lmax * pow((double)r, -beta));
        if (l < 1.0) l = 1.0;
        if (l > (double)n) l = (double)n;
        len[perm[r - 1]] = (int32_t)l;
    }
    gen_csr *g = calloc(1, sizeof(gen_csr));
    g->m = m; g->n = n;
    g->rowptr = malloc(sizeof(int32_t) * (size_t)(m + 1));
    int64_t nnz = 0;
    g->rowptr[0] = 0;
    for (int64_t i = 0; i < m; i++) { nnz += len[i]; g->rowptr[i + 1] = (int32_t)nnz; }
    g->nnz = nnz;
    g->colidx = malloc(sizeof(int32_t) * (size_t)(nnz > 0 ? nnz : 1));
    g->vals = malloc(sizeof(double) * (size_t)(nnz > 0 ? nnz : 1));
    unsigned char *mark = calloc((size_t)(n > 0 ? n : 1), 1);
    if (!g->colidx || !g->vals || !mark) { gen_free(g); free(mark); free(len); free(perm); return NULL; }
    for (int64_t i = 0; i < m; i++) {
        int32_t L = len[i];
        int32_t *c = g->colidx + g->rowptr[i];
        int32_t got = 0;
        uint64_t ctr = (uint64_t)g->rowptr[i];
        for (int64_t j = n - L; j < n; j++) {
            uint64_t r = rng(seed, 2, ctr++);
            int64_t tt = (int64_t)(((unsigned __int128)r * (unsigned __int128)(j + 1)) >> 64);
            int64_t pick = mark[tt] ? j : tt;
            mark[pick] = 1;
            c[got++] = (int32_t)pick;
        }
        /* sort ascending (insertion sort for short rows, qsort otherwise) */
        if (L <= 32) {
            for (int32_t a = 1; a < L; a++) {
                int32_t v = c[a], b = a - 1;
                while (b >= 0 && c[b] > v) { c[b + 1] = c[b]; b--; }
                c[b + 1] = v;
            }
        } else {
            qsort(c, (size_t)L, sizeof(int32_t), cmp_i32);
        }
        for (int32_t a = 0; a < L; a++) mark[c[a]] = 0;
    }
    for (int64_t k = 0; k < nnz; k++) g->vals[k] = u11(seed, 3, (uint64_t)k);
    free(mark); free(len); free(perm);
    return g;
}


/* 27-point Laplacian on an N^3 grid, Dirichlet truncation (reading R19):
 * row i = x + N*(y + N*z); centre 26, in-domain neighbours -1; columns
 * ascending.  nnz = (3N-2)^3.                                              */
gen_csr *gen_stencil27(int64_t N)
{
    int64_t m = N * N * N;
    int64_t nnz = (3 * N - 2) * (3 * N - 2) * (3 * N - 2);
    if (N <= 0) { m = 0; nnz = 0; }
    gen_csr *g = calloc(1, sizeof(gen_csr));
    g->m = m; g->n = m; g->nnz = nnz;
    g->rowptr = malloc(sizeof(int32_t) * (size_t)(m + 1));
    g->colidx = malloc(sizeof(int32_t) * (size_t)(nnz > 0 ? nnz : 1));
    g->vals = malloc(sizeof(double) * (size_t)(nnz > 0 ? nnz : 1));
    if (!g->rowptr || !g->colidx || !g->vals) { gen_free(g); return NULL; }
    int64_t o = 0;
    g->rowptr[0] = 0;
    for (int64_t z = 0; z < N; z++)
        for (int64_t y = 0; y < N; y++)
            for (int64_t x = 0; x < N; x++) {
                for (int dz = -1; dz <= 1; dz++) {
                    int64_t zz = z + dz;
                    if (zz < 0 || zz >= N) continue;
                    for (int dy = -1; dy <= 1; dy++) {
                        int64_t yy = y + dy;
                        if (yy < 0 || yy >= N) continue;
                        for (int dx = -1; dx <= 1; dx++) {
                            int64_t xx = x + dx;
                            if (xx < 0 || xx >= N) continue;
                            g->colidx[o] = (int32_t)(xx + N * (yy + N * zz));
                            g->vals[o] = (dx == 0 && dy == 0 && dz == 0) ? 26.0 : -1.0;
                            o++;
                        }
                    }
                }
                g->rowptr[x + N * (y + N * z) + 1] = (int32_t)o;
            }
    return g;
}

/* 1-D Laplacian tridiag(-1, 2, -1), Dirichlet, n rows. */
gen_csr *gen_laplace1d(int64_t n)
{
    int64_t nnz = n > 0 ? 3 * n - 2 : 0;
    gen_csr *g = calloc(1, sizeof(gen_csr));
    g->m = n; g->n = n; g->nnz = nnz;
    g->rowptr = malloc(sizeof(int32_t) * (size_t)(n + 1));
    g->colidx = malloc(sizeof(int32_t) * (size_t)(nnz > 0 ? nnz : 1));
    g->vals = malloc(sizeof(double) * (size_t)(nnz > 0 ? nnz : 1));
    int64_t o = 0;
    g->rowptr[0] = 0;
    for (int64_t i = 0; i < n; i++) {
        if (i > 0) { g->colidx[o] = (int32_t)(i - 1); g->vals[o++] = -1.0; }
        g->colidx[o] = (int32_t)i; g->vals[o++] = 2.0;
        if (i < n - 1) { g->colidx[o] = (int32_t)(i + 1); g->vals[o++] = -1.0; }
        g->rowptr[i + 1] = (int32_t)o;
    }
    return g;
}

/* ----------------------------------------------------------------------- */
/* NAS IS keys [ext:NPB-IS] create_seq(seed=314159265, a=1220703125):
 *   k = max_key/4;  key[i] = (int)(k * (u1 + u2 + u3 + u4)),
 * four consecutive randlc draws per key, summed left to right in double
 * (k is a power of two, so k*x is exact and the truncation is NPB's).       */
void gen_is_keys(int64_t n, int64_t max_key, uint64_t seed, uint64_t a, int32_t *keys)
{
    uint64_t s = seed;
    const double k = (double)(max_key / 4);
    for (int64_t i = 0; i < n; i++) {
        double x = randlc(&s, a);
        x += randlc(&s, a);
        x += randlc(&s, a);
        x += randlc(&s, a);
        keys[i] = (int32_t)(k * x);
    }
}

/* Parboil-histo-shaped image (reading R32; the paper's histo input is not
 * described): npix values in [0, nbins).  With probability 5/8 a pixel sits
 * near one of `hot` seeded centres (offset = sum of two uniform integers in
 * [-8, 8], triangular, wrapped into range) -- the hot spots that make the
 * saturating uint8 counters of Parboil histo matter; otherwise uniform.
 * splitmix64 streams: 11 = centres, 12 = per-pixel draws.                   */
void gen_histo_image(int64_t npix, int64_t nbins, int32_t hot, uint64_t seed, int32_t *img)
{
    if (hot < 1) hot = 1;
    int64_t *cen = (int64_t *)malloc(sizeof(int64_t) * (size_t)hot);
    for (int32_t h = 0; h < hot; h++) cen[h] = (int64_t)(rng(seed, 11, (uint64_t)h) % (uint64_t)nbins);
    for (int64_t i = 0; i < npix; i++) {
        uint64_t r = rng(seed, 12, (uint64_t)i);
        int64_t v;
        if ((r & 7) < 5) {
            int64_t c = cen[(r >> 3) % (uint64_t)hot];
            int64_t o = (int64_t)((r >> 24) % 17) + (int64_t)((r >> 40) % 17) - 16;
            v = ((c + o) % nbins + nbins) % nbins;
        } else {
            v = (int64_t)((r >> 8) % (uint64_t)nbins);
        }
        img[i] = (int32_t)v;
    }
    free(cen);
}
