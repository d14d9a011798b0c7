/*
 * swgen/swgen.c -- seeded synthetic protein sequences for tests and bench.
 *
 * Holds NONE of the method's arithmetic (no scoring, no alignment): it only
 * draws residues and lengths.  Both the oracle side (tests) and the product
 * side (tests, bench) consume its output; it imports neither.
 *
 * Counter-based: every random number is hash(seed, stream, a, b), so any
 * sequence can be regenerated alone from (seed, id) -- needed for sampled
 * parity at TrEMBL scale.
 *
 * Residue codes are 0..19 = "ARNDCQEGHILKMFPSTWYV" (NCBI order, first 20).
 */
#include <stdint.h>
#include <math.h>
#include <string.h>

enum { ST_LEN = 1, ST_RES = 2, ST_QRES = 3, ST_MUT = 5 };

static inline uint64_t smix(uint64_t z)
{
    z += 0x9E3779B97F4A7C15ull;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}

static inline uint64_t ctr(uint64_t seed, uint64_t stream, uint64_t a, uint64_t b)
{
    return smix(smix(smix(seed * 0x2545F4914F6CDD1Dull + stream) ^ a) + b);
}

static inline double u01(uint64_t x) { return (double)(x >> 11) * (1.0 / 9007199254740992.0); }

/* Swiss-Prot background composition (percent), ARNDCQEGHILKMFPSTWYV. */
static const double FREQ[20] = {8.25, 5.53, 4.06, 5.46, 1.38, 3.93, 6.72, 7.07, 2.27, 5.91,
                                9.65, 5.80, 2.41, 3.86, 4.74, 6.64, 5.35, 1.10, 2.92, 6.86};
static double CUM[20];
static int cum_ready = 0;

static void init_cum(void)
{
    double s = 0, c = 0;
    int k;
    if (cum_ready) return;
    for (k = 0; k < 20; ++k) s += FREQ[k];
    for (k = 0; k < 20; ++k) { c += FREQ[k] / s; CUM[k] = c; }
    CUM[19] = 1.0;
    cum_ready = 1;
}

static inline uint8_t residue(double u)
{
    int k = 0;
    while (k < 19 && u >= CUM[k]) ++k;
    return (uint8_t)k;
}

/*
 * Length of DB sequence `id`.
 *   kind 0 ("swissprot"): lognormal(mu, sigma) body plus a Pareto tail
 *          (fraction tail_frac, x_min 3000, alpha 1.6), clipped to [lmin, lmax].
 *   kind 1 ("tail"):      Pareto(x_min 3000 + 1, alpha 1.6) only, clipped.
 */
int64_t swgen_db_length(uint64_t seed, int64_t id, int32_t kind, double mu, double sigma,
                        double tail_frac, int64_t lmin, int64_t lmax)
{
    double u0 = u01(ctr(seed, ST_LEN, (uint64_t)id, 0));
    double u1 = u01(ctr(seed, ST_LEN, (uint64_t)id, 1));
    double u2 = u01(ctr(seed, ST_LEN, (uint64_t)id, 2));
    double L;
    if (kind == 1 || u0 < tail_frac) {
        L = 3001.0 * pow(1.0 - u1, -1.0 / 1.6);
    } else {
        double z = sqrt(-2.0 * log(1.0 - u1)) * cos(6.283185307179586 * u2);
        L = exp(mu + sigma * z);
    }
    if (L < (double)lmin) L = (double)lmin;
    if (L > (double)lmax) L = (double)lmax;
    return (int64_t)L;
}

void swgen_db_lengths(uint64_t seed, int64_t n, int32_t kind, double mu, double sigma,
                      double tail_frac, int64_t lmin, int64_t lmax, int64_t *out)
{
    int64_t i;
#pragma omp parallel for schedule(static)
    for (i = 0; i < n; ++i) out[i] = swgen_db_length(seed, i, kind, mu, sigma, tail_frac, lmin, lmax);
}

/* i.i.d. residues for `len` positions of sequence `id` in stream `stream`. */
static void fill_iid(uint64_t seed, uint64_t stream, int64_t id, int64_t len, uint8_t *dst)
{
    int64_t p;
    for (p = 0; p < len; ++p) dst[p] = residue(u01(ctr(seed, stream, (uint64_t)id, (uint64_t)p)));
}

/*
 * Fill the residues of DB sequences [0, n) at codes[off[i] .. off[i+1]).
 * Sequences whose plant_src[i] >= 0 are NOT touched (filled by swgen_mutate).
 */
void swgen_db_fill(uint64_t seed, int64_t n, const int64_t *off, const int32_t *plant_src, uint8_t *codes)
{
    int64_t i;
    init_cum();
#pragma omp parallel for schedule(dynamic, 1024)
    for (i = 0; i < n; ++i) {
        if (plant_src && plant_src[i] >= 0) continue;
        fill_iid(seed, ST_RES, i, off[i + 1] - off[i], codes + off[i]);
    }
}

void swgen_query_fill(uint64_t seed, int64_t nq, const int64_t *off, uint8_t *codes)
{
    int64_t i;
    init_cum();
    for (i = 0; i < nq; ++i) fill_iid(seed, ST_QRES, i, off[i + 1] - off[i], codes + off[i]);
}

/*
 * Mutant of a source sequence (planted homolog).  Walks the source left to
 * right; per position, with probability p_sub substitute a random residue, with
 * probability p_indel/2 delete 1-3 residues, with p_indel/2 insert 1-3 random
 * residues after it.  Deterministic in (seed, key).  If dst is NULL only the
 * length is returned; else writes at most cap residues and returns the length.
 */
int64_t swgen_mutate(uint64_t seed, uint64_t key, const uint8_t *src, int64_t len,
                     double p_sub, double p_indel, uint8_t *dst, int64_t cap)
{
    int64_t p = 0, o = 0, r = 0;
    init_cum();
    while (p < len) {
        double u = u01(ctr(seed, ST_MUT, key, (uint64_t)r++));
        if (u < p_indel * 0.5) {                       /* deletion of 1..3 */
            int64_t k = 1 + (int64_t)(u01(ctr(seed, ST_MUT, key, (uint64_t)r++)) * 3.0);
            p += k;
            continue;
        }
        {
            uint8_t c = src[p];
            if (u01(ctr(seed, ST_MUT, key, (uint64_t)r++)) < p_sub)
                c = residue(u01(ctr(seed, ST_MUT, key, (uint64_t)r++)));
            if (dst && o < cap) dst[o] = c;
            ++o;
        }
        if (u >= p_indel * 0.5 && u < p_indel) {       /* insertion of 1..3 */
            int64_t k = 1 + (int64_t)(u01(ctr(seed, ST_MUT, key, (uint64_t)r++)) * 3.0), t;
            for (t = 0; t < k; ++t) {
                uint8_t c = residue(u01(ctr(seed, ST_MUT, key, (uint64_t)r++)));
                if (dst && o < cap) dst[o] = c;
                ++o;
            }
        }
        ++p;
    }
    return o;
}
