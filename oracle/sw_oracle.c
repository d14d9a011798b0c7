/*
 * oracle/sw_oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * Plain, slow, obviously-correct CPU oracle for the hot path of SWDUAL
 * (Kedad-Sidhoum et al., ICPP 2014): Smith-Waterman local-alignment scoring
 * with affine gaps (Gotoh), score only, one int32 per (query, subject) pair.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl
 * reference legs may load this file's shared object.  The product library
 * (paper_conf_icpp_kedad_sidhoummmmt14_b200/) shares no code, header, table or
 * constant with it, and never calls it.
 *
 * What it computes (PAPER.md, /root/reference/PAPER.md):
 *   - L127-136 (sec. II.A): the score of an alignment is the sum of its column
 *     scores; "the maximal score is called the similarity".
 *   - L149-158 (sec. II.B): s (|s| = m, rows i) is compared with t (|t| = n,
 *     columns j); "the first row and column are filled with zeros";
 *     S_{i,j} is the similarity score of elements i and j.
 *   - L170-194 (sec. II.B, Eqs. (2)-(4), Gotoh):
 *         H_{i,j} = max( H_{i-1,j-1} + S_{i,j}, E_{i,j}, F_{i,j}, 0 )       (2)
 *         E_{i,j} = -Ge + max( E_{i,j-1}, H_{i,j-1} - Gs )                   (3)
 *         F_{i,j} = -Ge + max( F_{i-1,j}, H_{i-1,j} - Gs )                   (4)
 *     so a gap of length k costs Gs + k*Ge (reading R-1).
 *   - Borders: H_{0,j} = H_{i,0} = 0 (L153-154); E_{i,0} = F_{0,j} = -infinity
 *     (reading R-2: the paper only fixes H's borders; any value <= 0
 *     gives the same scores).
 *   - Result: max over all cells of H (the 0 in Eq. (2) makes it >= 0).
 *
 * Arithmetic: exact int32.  NEG stands for -infinity; it is far enough from
 * INT32_MIN that NEG - Gs - Ge cannot wrap for the penalties the tests use
 * (Gs, Ge <= 2^20).  S is indexed S[query letter][subject letter], row-major,
 * alpha x alpha int32.  Linear space: only row i-1 and row i of H, E, F are kept
 * (the values are the same as in the (m+1) x (n+1) matrices of L151-152).
 */
#include <stdint.h>
#include <stdlib.h>

#define NEG (INT32_MIN / 4)

static int32_t max2(int32_t a, int32_t b) { return a > b ? a : b; }

/* Score of one pair.  Returns -1 on allocation failure or a code >= alpha. */
int32_t oracle_gotoh_score(const uint8_t *s, int64_t m,
                           const uint8_t *t, int64_t n,
                           const int32_t *S, int32_t alpha,
                           int32_t Gs, int32_t Ge)
{
    int64_t i, j;
    int32_t best = 0;
    int32_t *Hprev, *Hcur, *Eprev, *Ecur, *Fprev, *Fcur, *tmp;
    if (m <= 0 || n <= 0) return 0;                       /* empty alignment only */
    Hprev = (int32_t *)malloc(sizeof(int32_t) * (size_t)(n + 1));
    Hcur  = (int32_t *)malloc(sizeof(int32_t) * (size_t)(n + 1));
    Eprev = (int32_t *)malloc(sizeof(int32_t) * (size_t)(n + 1));
    Ecur  = (int32_t *)malloc(sizeof(int32_t) * (size_t)(n + 1));
    Fprev = (int32_t *)malloc(sizeof(int32_t) * (size_t)(n + 1));
    Fcur  = (int32_t *)malloc(sizeof(int32_t) * (size_t)(n + 1));
    if (!Hprev || !Hcur || !Eprev || !Ecur || !Fprev || !Fcur) { best = -1; goto done; }

    /* row 0: H_{0,j} = 0, E/F = -inf */
    for (j = 0; j <= n; ++j) { Hprev[j] = 0; Eprev[j] = NEG; Fprev[j] = NEG; }

    for (i = 1; i <= m; ++i) {
        if (s[i - 1] >= alpha) { best = -1; goto done; }
        /* column 0: H_{i,0} = 0, E_{i,0} = -inf */
        Hcur[0] = 0; Ecur[0] = NEG; Fcur[0] = NEG;
        for (j = 1; j <= n; ++j) {
            int32_t Sij, h;
            if (t[j - 1] >= alpha) { best = -1; goto done; }
            Sij = S[(int64_t)s[i - 1] * alpha + t[j - 1]];
            Ecur[j] = -Ge + max2(Ecur[j - 1], Hcur[j - 1] - Gs);          /* Eq. (3) */
            Fcur[j] = -Ge + max2(Fprev[j],   Hprev[j]   - Gs);            /* Eq. (4) */
            h = max2(max2(Hprev[j - 1] + Sij, Ecur[j]), max2(Fcur[j], 0)); /* Eq. (2) */
            Hcur[j] = h;
            if (h > best) best = h;
        }
        tmp = Hprev; Hprev = Hcur; Hcur = tmp;
        tmp = Eprev; Eprev = Ecur; Ecur = tmp;
        tmp = Fprev; Fprev = Fcur; Fcur = tmp;
    }
done:
    free(Hprev); free(Hcur); free(Eprev); free(Ecur); free(Fprev); free(Fcur);
    return best;
}

/*
 * Many-query x database (L196-201: "compare a set q of m query sequences to a
 * set d of n database sequences").  Sequences are concatenated code arrays with
 * offsets (sequence k = codes[off[k] .. off[k+1])).  Pairs are scored one after
 * the other, in order; scores is [nq][nd] row-major.  Subset [d_begin, d_end)
 * of the database is scored so that callers can split the work across
 * processes.  Returns 0, or -1 if any pair failed.
 */
int32_t oracle_gotoh_search(const uint8_t *qcodes, const int64_t *qoff, int64_t nq,
                            const uint8_t *dcodes, const int64_t *doff, int64_t nd,
                            int64_t d_begin, int64_t d_end,
                            const int32_t *S, int32_t alpha, int32_t Gs, int32_t Ge,
                            int32_t *scores)
{
    int64_t a, b;
    int32_t rc = 0;
    for (a = 0; a < nq; ++a) {
        for (b = d_begin; b < d_end && b < nd; ++b) {
            int32_t v = oracle_gotoh_score(qcodes + qoff[a], qoff[a + 1] - qoff[a],
                                           dcodes + doff[b], doff[b + 1] - doff[b],
                                           S, alpha, Gs, Ge);
            if (v < 0) rc = -1;
            scores[a * nd + b] = v;
        }
    }
    return rc;
}

/*
 * Best local alignment of one pair: its end cell, start cell and path
 * (the traceback keeps "the cell that was
 * used to produce the value" of each matrix element).  Plain full matrices
 * H, E, F of size (m+1) x (n+1) (L151-152), Eqs. (2)-(4) unclamped, then a
 * traceback.  Where the paper is silent (reading R-13):
 *   - end cell: the cell with the maximal H; ties -> smallest j (subject
 *     position), then smallest i (query position);
 *   - traceback, state H at (i, j): stop if H == 0; else the diagonal if
 *     H == H_{i-1,j-1} + S_ij, else E if H == E_ij, else F;
 *   - state E (a gap in the query, consuming subject residue j): back to H at
 *     (i, j-1) if E_ij == H_{i,j-1} - Gs - Ge (opening preferred on a tie), else
 *     stay in E; state F likewise along i;
 *   - coordinates 0-based and inclusive: the alignment covers s[q_begin..q_end]
 *     and t[d_begin..d_end]; a zero score has no alignment (all four = -1).
 * ops: run-length codes (len << 2 | op), op 0 = M (aligned pair), 1 = I (query
 * residue against a gap, F), 2 = D (subject residue against a gap, E), from the
 * start of the alignment to its end.
 * out5 = {score, q_begin, q_end, d_begin, d_end}.  Returns the number of ops,
 * -1 on allocation failure / bad code, -2 if ops_cap is too small.
 */
int32_t oracle_gotoh_align(const uint8_t *s, int64_t m, const uint8_t *t, int64_t n,
                           const int32_t *S, int32_t alpha, int32_t Gs, int32_t Ge,
                           int32_t *out5, uint32_t *ops, int32_t ops_cap)
{
    int64_t i, j, W = n + 1, bi = 0, bj = 0;
    int32_t best = 0, nops = 0, rc = 0;
    int32_t *H = NULL, *E = NULL, *F = NULL;
    uint32_t *rev = NULL;
    out5[0] = 0; out5[1] = out5[2] = out5[3] = out5[4] = -1;
    if (m <= 0 || n <= 0) return 0;
    H = (int32_t *)malloc(sizeof(int32_t) * (size_t)((m + 1) * W));
    E = (int32_t *)malloc(sizeof(int32_t) * (size_t)((m + 1) * W));
    F = (int32_t *)malloc(sizeof(int32_t) * (size_t)((m + 1) * W));
    rev = (uint32_t *)malloc(sizeof(uint32_t) * (size_t)(m + n + 1));
    if (!H || !E || !F || !rev) { rc = -1; goto done; }
    for (j = 0; j <= n; ++j) { H[j] = 0; E[j] = NEG; F[j] = NEG; }
    for (i = 1; i <= m; ++i) {
        if (s[i - 1] >= alpha) { rc = -1; goto done; }
        H[i * W] = 0; E[i * W] = NEG; F[i * W] = NEG;
        for (j = 1; j <= n; ++j) {
            int32_t Sij, h;
            if (t[j - 1] >= alpha) { rc = -1; goto done; }
            Sij = S[(int64_t)s[i - 1] * alpha + t[j - 1]];
            E[i * W + j] = -Ge + max2(E[i * W + j - 1], H[i * W + j - 1] - Gs);        /* Eq. (3) */
            F[i * W + j] = -Ge + max2(F[(i - 1) * W + j], H[(i - 1) * W + j] - Gs);    /* Eq. (4) */
            h = max2(max2(H[(i - 1) * W + j - 1] + Sij, E[i * W + j]), max2(F[i * W + j], 0)); /* (2) */
            H[i * W + j] = h;
            /* end-cell tie-break: smallest j, then smallest i */
            if (h > best || (h == best && h > 0 && (j < bj || (j == bj && i < bi)))) { best = h; bi = i; bj = j; }
        }
    }
    out5[0] = best;
    if (best == 0) goto done;
    {
        int state = 0;  /* 0 = H, 1 = E, 2 = F */
        int32_t run_op = -1, run_len = 0;
        i = bi; j = bj;
        for (;;) {
            int32_t op;
            if (state == 0) {
                int32_t h = H[i * W + j];
                if (h == 0) break;
                if (h == H[(i - 1) * W + j - 1] + S[(int64_t)s[i - 1] * alpha + t[j - 1]]) {
                    op = 0; --i; --j;
                } else if (h == E[i * W + j]) { state = 1; continue; }
                else { state = 2; continue; }
            } else if (state == 1) {
                op = 2;
                state = (E[i * W + j] == H[i * W + j - 1] - Gs - Ge) ? 0 : 1;
                --j;
            } else {
                op = 1;
                state = (F[i * W + j] == H[(i - 1) * W + j] - Gs - Ge) ? 0 : 2;
                --i;
            }
            if (op == run_op) ++run_len;
            else {
                if (run_len) rev[nops++] = ((uint32_t)run_len << 2) | (uint32_t)run_op;
                run_op = op; run_len = 1;
            }
        }
        if (run_len) rev[nops++] = ((uint32_t)run_len << 2) | (uint32_t)run_op;
        out5[1] = (int32_t)i; out5[2] = (int32_t)(bi - 1);
        out5[3] = (int32_t)j; out5[4] = (int32_t)(bj - 1);
        if (nops > ops_cap) { rc = -2; goto done; }
        for (int32_t k = 0; k < nops; ++k) ops[k] = rev[nops - 1 - k];
        rc = nops;
    }
done:
    free(H); free(E); free(F); free(rev);
    return rc;
}
