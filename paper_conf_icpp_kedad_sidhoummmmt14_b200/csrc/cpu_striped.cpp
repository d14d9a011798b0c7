// CPU-type processing element of the hybrid SWDUAL (PAPER.md
// sec. III: tasks run on "m CPUs and k GPUs", L309-350; the paper's CPU workers
// run a SIMD Smith-Waterman, L529-539).  Product code, compiled with -mavx2:
// the striped query-profile method (one query against one DB sequence at a
// time, 16 int16 lanes per AVX2 register, the query cut into 16 interleaved
// segments of segLen rows: row r lives in lane r / segLen, vector r % segLen),
// with the lazy-F pass that carries the vertical gap across lane boundaries.
//
// Values are kept relu-clamped at 0 exactly like the GPU kernels (DESIGN.md
// R-9: E, F, H >= 0 loses nothing because H's 0-floor absorbs negatives) in
// saturating int16; a pair whose maximum reaches 32767 - S_max is re-scored by
// the scalar int32 recurrence below (the first saturation needs an earlier,
// exact H >= 32768 - S_max, which already raised the maximum).
#include <immintrin.h>

#include <algorithm>
#include <atomic>
#include <cstdint>
#include <cstring>
#include <thread>
#include <vector>

namespace swdual {

namespace {

constexpr int LANES = 16;

// lane l <- lane l-1, lane 0 <- 0 (across the two 128-bit halves)
inline __m256i shift_lanes_up(__m256i v) {
  const __m256i lo_to_hi = _mm256_permute2x128_si256(v, v, 0x08);  // [0, v.lo]
  return _mm256_alignr_epi8(v, lo_to_hi, 14);
}

inline int16_t hmax16(__m256i v) {
  __m128i m = _mm_max_epi16(_mm256_castsi256_si128(v), _mm256_extracti128_si256(v, 1));
  m = _mm_max_epi16(m, _mm_srli_si128(m, 8));
  m = _mm_max_epi16(m, _mm_srli_si128(m, 4));
  m = _mm_max_epi16(m, _mm_srli_si128(m, 2));
  return int16_t(_mm_extract_epi16(m, 0));
}

// Scalar int32 Gotoh (Eqs. (2)-(4), E/F clamped at 0) for flagged pairs.
int32_t score_s32(const uint8_t* q, int64_t m, const uint8_t* d, int64_t n, const int8_t* S, int alpha, int32_t Gs,
                  int32_t Ge, std::vector<int32_t>& H, std::vector<int32_t>& F) {
  H.assign(size_t(n + 1), 0);
  F.assign(size_t(n + 1), 0);
  int32_t best = 0;
  for (int64_t i = 1; i <= m; ++i) {
    const int8_t* row = S + int64_t(q[i - 1]) * alpha;
    int32_t diag = 0, left = 0, E = 0;
    for (int64_t j = 1; j <= n; ++j) {
      E = std::max({E - Ge, left - Gs - Ge, 0});
      F[size_t(j)] = std::max({F[size_t(j)] - Ge, H[size_t(j)] - Gs - Ge, 0});
      const int32_t h = std::max({diag + row[d[j - 1]], E, F[size_t(j)], 0});
      diag = H[size_t(j)];
      H[size_t(j)] = h;
      left = h;
      best = std::max(best, h);
    }
  }
  return best;
}

struct alignas(32) Vec {
  __m256i v;
};
static_assert(sizeof(Vec) == sizeof(__m256i), "Vec must be one register");

struct Striped {
  int segLen = 0;
  std::vector<Vec> prof;  // [alpha][segLen]
  std::vector<Vec> h0, h1, e;
};

void build_profile(Striped& P, const uint8_t* q, int64_t m, const int8_t* S, int alpha) {
  P.segLen = int((m + LANES - 1) / LANES);
  P.prof.assign(size_t(alpha) * size_t(P.segLen), Vec{_mm256_setzero_si256()});
  for (int a = 0; a < alpha; ++a)
    for (int k = 0; k < P.segLen; ++k) {
      alignas(32) int16_t v[LANES];
      for (int l = 0; l < LANES; ++l) {
        const int64_t r = int64_t(l) * P.segLen + k;
        v[l] = r < m ? int16_t(S[int64_t(q[r]) * alpha + a]) : int16_t(-64);  // padded rows (R-12)
      }
      P.prof[size_t(a) * size_t(P.segLen) + size_t(k)].v = _mm256_load_si256(reinterpret_cast<const __m256i*>(v));
    }
  P.h0.assign(size_t(P.segLen), Vec{_mm256_setzero_si256()});
  P.h1.assign(size_t(P.segLen), Vec{_mm256_setzero_si256()});
  P.e.assign(size_t(P.segLen), Vec{_mm256_setzero_si256()});
}

int16_t score_striped(Striped& P, const uint8_t* d, int64_t n, int16_t gsge, int16_t ge) {
  const int segLen = P.segLen;
  const __m256i zero = _mm256_setzero_si256();
  const __m256i vGapO = _mm256_set1_epi16(gsge);
  const __m256i vGapE = _mm256_set1_epi16(ge);
  __m256i* Hs = &P.h0.data()->v;
  __m256i* Hl = &P.h1.data()->v;
  __m256i* E = &P.e.data()->v;
  for (int k = 0; k < segLen; ++k) { Hs[k] = zero; E[k] = zero; }
  __m256i vMax = zero;
  for (int64_t j = 0; j < n; ++j) {
    const __m256i* pr = &P.prof[size_t(d[j]) * size_t(segLen)].v;
    __m256i vF = zero;
    __m256i vH = shift_lanes_up(Hs[segLen - 1]);  // H_{r-1, j-1} for the rows at k = 0
    std::swap(Hs, Hl);
    for (int k = 0; k < segLen; ++k) {
      vH = _mm256_adds_epi16(vH, pr[k]);           // H_{i-1,j-1} + S_ij
      const __m256i e = E[k];
      vH = _mm256_max_epi16(vH, e);                // Eq. (2)
      vH = _mm256_max_epi16(vH, vF);
      vH = _mm256_max_epi16(vH, zero);
      vMax = _mm256_max_epi16(vMax, vH);
      Hs[k] = vH;
      const __m256i ho = _mm256_subs_epi16(vH, vGapO);
      E[k] = _mm256_max_epi16(_mm256_max_epi16(_mm256_subs_epi16(e, vGapE), ho), zero);  // Eq. (3), next column
      vF = _mm256_max_epi16(_mm256_max_epi16(_mm256_subs_epi16(vF, vGapE), ho), zero);   // Eq. (4), next row
      vH = Hl[k];
    }
    // Lazy F: the vertical gaps that cross from the last row of lane l-1 into
    // lane l.  Propagated candidate F^p enters row k; the true F is max(F^main,
    // F^p) and H rises to F^p where it is larger.  Stop once no lane's next
    // candidate beats max(H^main - Gs - Ge, 0) (<= F^main of the next row).
    vF = shift_lanes_up(vF);
    for (int k = 0;;) {
      const __m256i hm = Hs[k];
      const __m256i hn = _mm256_max_epi16(hm, vF);
      Hs[k] = hn;
      vMax = _mm256_max_epi16(vMax, hn);
      E[k] = _mm256_max_epi16(E[k], _mm256_subs_epi16(hn, vGapO));  // E_{i,j+1} sees the raised H
      vF = _mm256_max_epi16(_mm256_subs_epi16(vF, vGapE), zero);
      // relu domain: F^main of the next row is >= max(H^main - Gs - Ge, 0)
      const __m256i gt = _mm256_cmpgt_epi16(vF, _mm256_max_epi16(_mm256_subs_epi16(hm, vGapO), zero));
      if (_mm256_testz_si256(gt, gt)) break;
      if (++k == segLen) {
        k = 0;
        vF = shift_lanes_up(vF);
      }
    }
  }
  return hmax16(vMax);
}

}  // namespace

// Score n_queries x n_seqs pairs on n_threads host threads (DB sequences dealt
// dynamically in chunks).  Inputs validated by the caller (engine.cpp).
void cpu_search_avx2(const uint8_t* qcodes, const int64_t* qoff, int32_t nq, const uint8_t* dcodes,
                     const int64_t* doff, int64_t n_seqs, int alpha, const int8_t* S, int32_t Gs, int32_t Ge,
                     int32_t n_threads, int32_t* scores) {
  int smax = -128;
  for (int i = 0; i < alpha * alpha; ++i) smax = std::max<int>(smax, S[i]);
  const int32_t thr = smax > 0 ? 32767 - smax : 32767;
  const bool s16 = Gs + Ge <= 32767;
  for (int32_t qi = 0; qi < nq; ++qi) {
    const uint8_t* q = qcodes + (qoff[qi] - qoff[0]);
    const int64_t m = qoff[qi + 1] - qoff[qi];
    int32_t* out = scores + int64_t(qi) * n_seqs;
    std::atomic<int64_t> next{0};
    const int64_t chunk = 64;
    auto worker = [&]() {
      Striped P;
      std::vector<int32_t> H, F;
      if (m > 0) build_profile(P, q, m, S, alpha);
      for (;;) {
        const int64_t b = next.fetch_add(chunk);
        if (b >= n_seqs) break;
        const int64_t e = std::min(n_seqs, b + chunk);
        for (int64_t d = b; d < e; ++d) {
          const int64_t n = doff[d + 1] - doff[d];
          const uint8_t* t = dcodes + (doff[d] - doff[0]);
          if (m == 0 || n == 0) { out[d] = 0; continue; }
          int32_t v = s16 ? score_striped(P, t, n, int16_t(Gs + Ge), int16_t(std::min(Ge, 32767))) : thr;
          if (v >= thr) v = score_s32(q, m, t, n, S, alpha, Gs, Ge, H, F);
          out[d] = v;
        }
      }
    };
    const int nt = std::max(1, n_threads);
    if (nt == 1) {
      worker();
    } else {
      std::vector<std::thread> pool;
      for (int t = 0; t < nt; ++t) pool.emplace_back(worker);
      for (auto& th : pool) th.join();
    }
  }
}

}  // namespace swdual
