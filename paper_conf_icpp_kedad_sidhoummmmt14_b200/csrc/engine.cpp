// Host engine and C ABI of the SWDUAL hot path (include/swdual.h).
//
//   sw_load_db : host packer -- validate codes, sort the
//                database by length (longest first, ties by index), pair
//                neighbours, interleave each pair column by column into 16-bit
//                words padded to 4 columns, upload stream + pair table once.
//   sw_search  : per query, build the int8 query profile on the device, launch
//                the inter-task DPX kernel over the short pairs and over the
//                long pairs, then the int32 re-score of flagged pairs; scores
//                land directly in the caller's DB order (un-permute fused into
//                the kernel epilogue).
#include <algorithm>
#include <atomic>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <new>
#include <stdexcept>
#include <numeric>
#include <string>
#include <thread>
#include <vector>

#include <cuda_runtime.h>

#include "../../include/swdual.h"
#include "sw_internal.h"

using namespace swdual;

namespace {

thread_local std::string g_tls_err;

struct DevBuf {
  void* p = nullptr;
  size_t n = 0;
  DevBuf() = default;
  DevBuf(const DevBuf&) = delete;
  DevBuf& operator=(const DevBuf&) = delete;
  ~DevBuf() { release(); }
  void release() {
    if (p) cudaFree(p);
    p = nullptr;
    n = 0;
  }
  cudaError_t ensure(size_t bytes) {
    if (bytes <= n && p) return cudaSuccess;
    // growing: an earlier search (on any stream) may still use the old buffer
    if (p) { cudaError_t e = cudaDeviceSynchronize(); if (e != cudaSuccess) return e; }
    release();
    size_t b = std::max<size_t>(bytes, 256);
    cudaError_t e = cudaMalloc(&p, b);
    if (e != cudaSuccess) { p = nullptr; return e; }
    n = b;
    return cudaSuccess;
  }
  template <class T> T* as() const { return reinterpret_cast<T*>(p); }
};

// Pinned staging of a search's host -> device uploads (queries, work-item tables).
// A cudaMemcpyAsync from pageable memory first waits for the stream to drain, so a
// search's host-side preparation would run while the GPU idles; from pinned memory
// the copies queue behind the previous search's kernels.  Two halves alternate
// between consecutive searches; a half is refilled only after the event recorded
// behind its last copy (two searches ago) has completed.
struct HostStage {
  struct Half {
    uint8_t* p = nullptr;
    size_t cap = 0, used = 0;
    cudaEvent_t ev = nullptr;
    bool pending = false;
    std::vector<uint8_t*> retired;  // outgrown buffers, freed once `ev` completes
  };
  Half half[2];
  int cur = 0;
  cudaError_t begin() {
    cur ^= 1;
    Half& H = half[cur];
    if (H.pending) {
      cudaError_t e = cudaEventSynchronize(H.ev);
      if (e != cudaSuccess) return e;
      H.pending = false;
    }
    for (uint8_t* q : H.retired) cudaFreeHost(q);
    H.retired.clear();
    H.used = 0;
    return cudaSuccess;
  }
  cudaError_t copy(void* dst, const void* src, size_t bytes, cudaStream_t st) {
    if (bytes == 0) return cudaSuccess;
    Half& H = half[cur];
    size_t off = (H.used + 15) & ~size_t(15);
    if (off + bytes > H.cap) {  // grow: earlier copies of this search may still read the old buffer
      const size_t cap = std::max<size_t>({2 * H.cap, off + bytes, size_t(1) << 20});
      uint8_t* q = nullptr;
      cudaError_t e = cudaMallocHost(&q, cap);
      if (e != cudaSuccess) return e;
      if (H.p) H.retired.push_back(H.p);
      H.p = q;
      H.cap = cap;
      off = 0;
    }
    if (!H.ev) {
      cudaError_t e = cudaEventCreateWithFlags(&H.ev, cudaEventDisableTiming);
      if (e != cudaSuccess) return e;
    }
    std::memcpy(H.p + off, src, bytes);
    H.used = off + bytes;
    cudaError_t e = cudaMemcpyAsync(dst, H.p + off, bytes, cudaMemcpyHostToDevice, st);
    if (e != cudaSuccess) return e;
    H.pending = true;
    return cudaEventRecord(H.ev, st);  // behind every copy: an early exit never leaves one unguarded
  }
  void release() {
    for (Half& H : half) {
      if (H.pending && H.ev) cudaEventSynchronize(H.ev);
      for (uint8_t* q : H.retired) cudaFreeHost(q);
      H.retired.clear();
      if (H.p) cudaFreeHost(H.p);
      if (H.ev) cudaEventDestroy(H.ev);
      H = Half{};
    }
  }
};

struct SwError {
  int32_t code;
  std::string msg;
};

#define SW_CK(call)                                                                          \
  do {                                                                                       \
    cudaError_t e_ = (call);                                                                 \
    if (e_ != cudaSuccess)                                                                   \
      throw SwError{e_ == cudaErrorMemoryAllocation ? SW_ENOMEM : SW_ECUDA,                  \
                    std::string(#call) + ": " + cudaGetErrorString(e_)};                     \
  } while (0)

[[noreturn]] void fail(int32_t code, const std::string& m) { throw SwError{code, m}; }

constexpr int T_LONG = 3000;
// A short item (one lane group, all strips of its query) may run at most
// max(CRIT_MIN_STEPS, CRIT_FRACTION x the average lane group's wavefront steps
// of the launch); longer (query, pair) work goes to the intra-task mode.
constexpr int64_t CRIT_MIN_STEPS = 16384;
constexpr double LINK_LAG_STEPS = 32;   // the long kernel's producer lead (kernels.cu LINK_LAG)
constexpr double CRIT_FRACTION = 0.35;  // pairs longer than this are launched separately

}  // namespace

struct sw_db_s;
struct sw_assembly_s;

struct sw_handle_s {
  int device = 0;
  int sms = 148;
  uint32_t flags = 0;
  std::string err;
  std::vector<sw_db_s*> dbs;
  std::vector<sw_assembly_s*> assemblies;
  // scratch (grown on demand)
  DevBuf qcodes, qoff, matrix, prof, bbuf1, bbuf0, wrap, counters, ovf, ovf_count, scores_tmp, rbuf, qdesc;
  DevBuf rgrows, rflags;  // re-score: CTA-to-CTA rows, counters
  DevBuf imap;            // short work item order (mode 1 items, then mode 0 items)
  DevBuf lmap;            // long work item order
  DevBuf vq, sinfo;       // packed mode-1 slots: strip-padded query codes per half, per-strip info
  HostStage stage;        // pinned staging of sw_search's uploads
  cudaStream_t side = nullptr;             // the long-pair kernel's stream when short pairs run too
  cudaEvent_t ev_fork = nullptr, ev_join = nullptr;

  cudaEvent_t ev_begin = nullptr, ev_end = nullptr;
  // the previous search's completion: a search on another stream waits for it on the
  // device, because both use this handle's scratch
  cudaEvent_t ev_done = nullptr;
  cudaStream_t done_stream = nullptr;
  bool done_valid = false;
  bool search_timed = false;
  bool timing_accumulate = false;
  std::vector<int> event_kind;
  // options
  int64_t opt_thr = 0, opt_G = 0, opt_R = 0;
  int64_t opt_t_long = -1;      // >= 0: pairs longer than this always use the intra-task mode
  int64_t opt_query_pairs = 1;  // pair queries two per register for the short pairs
  int64_t opt_pack_queries = 1; // mode-1 slots: fill the shorter half with further queries (strip-aligned)
  int64_t opt_bank_copy = 1;    // query-pair profile: second smem copy shifted by 64 B for odd lane groups
  int64_t opt_bank_skew = 1;    // mode-0 profile copies: per-copy bank skew (mode0_copies)
  int64_t opt_const_gaps = 1;   // gaps 10/2: the constant-gap kernel instantiations
  int64_t opt_nibble = 1;       // alphabets <= 15: 4-bit DB stream
  int64_t opt_small_ctas = 1;   // latency-bound single-query searches: 32-thread CTAs
  int64_t opt_rescore_rows = 0; // int32 re-score rows per lane: 0 = automatic (4 or 8), 4, 8
  int64_t opt_crit_min = CRIT_MIN_STEPS;                    // long-pair rule (see launch_all)
  int64_t opt_crit_pct = int64_t(CRIT_FRACTION * 100 + 0.5);
  int64_t opt_align_ws_mb = 2048;  // sw_align: traceback-code workspace per batch
  // sw_align scratch (separate from sw_search's: a search may still be running on another stream)
  DevBuf a_qcodes, a_qoff, a_matrix, a_items, a_links, a_trace, a_best, a_ops, a_out, a_counter;
  DevBuf a_submap, a_grows, a_gflags, a_partial, a_done;
  // last-search bookkeeping
  sw_stats_t stats{};
  cudaStream_t last_stream = nullptr;
  std::vector<std::pair<cudaEvent_t, cudaEvent_t>> events;
  size_t n_events_used = 0;
};

struct sw_db_s {
  sw_handle_s* h = nullptr;
  int64_t n_seqs = 0, n_res = 0;
  int alpha = 0;
  int64_t max_len = 0;
  std::vector<PairRec> pairs;    // host copy, sorted longest first
  std::vector<int64_t> seq_len;  // caller order
  std::vector<int64_t> sorted_lens;  // descending, non-empty only (for overflow bounds)
  int n_long = 0;                // pairs [0, n_long) have len > T_LONG
  int nib = 0;                   // 4-bit pair stream (alphabet <= 15)
  // per-DB constants of the pair table (computed once at load)
  double sum_short_len = 0, sum_long_len = 0, short_res = 0;
  int32_t max_short = 0, max_long = 0;
  std::vector<int64_t> len_prefix;  // [np+1] prefix of padded pair lengths
  std::vector<double> res_prefix;   // [np+1] prefix of real residues (both halves)
  DevBuf stream, dpairs;
  std::vector<int64_t> seq_loc;  // caller index -> 2 * pair + half (-1: empty); built on first sw_align
  // output mapping (sw_load_db_mapped): scores of sequence d land in column out_index[d] of
  // rows of out_n columns -- e.g. a rank's shard writing into rank 0's full matrix
  int64_t out_n = 0;
  bool mapped = false;
  DevBuf dcols;                  // mapped: this DB's output columns, zeroed in every query row per search
  int64_t n_cols = 0;
};

struct sw_assembly_s {
  sw_handle_s* h = nullptr;
  int n_blocks = 0;
  int64_t total = 0, src_need = 0, n_queries = 0, N = 0;
  DevBuf blocks, prefix, rows, cols;
};

static int32_t set_err(sw_handle_s* h, int32_t code, const std::string& m) {
  if (h) h->err = m;
  g_tls_err = m;
  return code;
}

template <class F>
static int32_t guarded(sw_handle_s* h, F&& f) {
  try {
    f();
    return SW_OK;
  } catch (const SwError& e) {
    return set_err(h, e.code, e.msg);
  } catch (const std::bad_alloc&) {
    return set_err(h, SW_ENOMEM, "host allocation failed");
  } catch (const std::exception& e) {
    return set_err(h, SW_EINVAL, e.what());
  }
}

// ----------------------------------------------------------------------------
// Bank-spread copies of the mode-0 (single-query) strip profile.  Lane k of a
// group loads its rows at copy + letter * LS + k * LB (+ the row unit, equal for
// all lanes), LS a multiple of 128 B, so only the copy decides which banks the
// lane groups of one shared-memory phase hit.  The width of that load is 8 B
// only when a sub-lane's rows are whole 8-row units (R = 16, 32), else 4 B, so a
// phase holds 128 / width / G groups.  With 2 to 4 such groups, each copy gets
// a per-copy skew (multiple of 4 B, exhaustive search) minimising the worst bank
// load of the phase -- conflict-free for every geometry; the previous linear
// layout (copy c at c * (SB + 128 / ncopy), sized for 8-byte loads) left 2-way
// conflicts at R = 8, 24 with G = 8, 16.  Otherwise the linear layout stays.
struct Mode0Copies { int ncopy, cstride; uint32_t skew; int bytes; };
static Mode0Copies mode0_copies(int G, int R, int LB, int SB, bool on, bool skewed) {
  Mode0Copies c{1, SB, 0u, SB};
  if (!on) return c;
  const int N = (R % 8 == 0) ? R / 2 : R;               // rows per sub-lane
  const int w = (R % 8 == 0 && N % 8 == 0) ? 8 : 4;     // bytes per lane per profile load
  const int gpp = std::max(1, (128 / w) / G);           // lane groups per phase
  if (!skewed || gpp > 4 || gpp < 2) {                  // linear layout (previous rule)
    c.ncopy = std::max(1, (128 / (R % 8 == 0 ? 8 : 4)) / G);
    c.cstride = SB + (c.ncopy > 1 ? 128 / c.ncopy : 0);
    c.bytes = (c.ncopy - 1) * c.cstride + SB;
    return c;
  }
  c.ncopy = gpp;
  c.cstride = (SB + 127) / 128 * 128 + 128;
  // exhaustive over the (up to 3) free skews, lexicographic; stops at conflict-free
  auto worst_of = [&](const int* sk) {
    int cnt[32] = {0}, wmax = 0;
    for (int q = 0; q < c.ncopy; ++q)
      for (int k = 0; k < G; ++k)
        for (int b = 0; b < w; b += 4) wmax = std::max(wmax, ++cnt[((sk[q] + k * LB + b) / 4) % 32]);
    return wmax;
  };
  int sk[4] = {0, 0, 0, 0}, best_sk[4] = {0, 0, 0, 0}, best = 1 << 30;
  const int n1 = c.ncopy > 1 ? 32 : 1, n2 = c.ncopy > 2 ? 32 : 1, n3 = c.ncopy > 3 ? 32 : 1;
  for (int i1 = 0; i1 < n1 && best > 1; ++i1)
    for (int i2 = 0; i2 < n2 && best > 1; ++i2)
      for (int i3 = 0; i3 < n3 && best > 1; ++i3) {
        sk[1] = 4 * i1; sk[2] = 4 * i2; sk[3] = 4 * i3;
        const int v = worst_of(sk);
        if (v < best) { best = v; std::copy(sk, sk + 4, best_sk); }
      }
  std::copy(best_sk, best_sk + 4, sk);
  for (int cp = 0; cp < c.ncopy; ++cp) c.skew |= uint32_t(sk[cp] / 4) << (8 * cp);
  c.bytes = (c.ncopy - 1) * c.cstride + sk[c.ncopy - 1] + SB;
  return c;
}

// geometry of the inter-task kernel for a query of m rows and a launch whose
// pairs average Lavg columns
// long = true: the intra-task (G = 32) unit-interleaved layout, LB = the unit
// (8 bytes, the lane's offset); otherwise lane blocks of an odd number of units,
// letters padded to a multiple of 128 B when bank-spread copies are used.
static ProfGeom make_geom(int G, int R, int m, int alpha, bool long_mode = false, bool pad128 = false) {
  ProfGeom g{};
  g.G = G;
  g.R = R;
  g.UB = (R % 8 == 0) ? 8 : 4;
  g.il = long_mode ? 1 : 0;
  g.LB = long_mode ? g.UB : ((R % 8 == 0) ? (((R / 8) | 1) * 8) : (((R / 4) | 1) * 4));
  g.LS = long_mode ? G * R : G * g.LB;
  if (pad128) g.LS = ((g.LS + 127) / 128) * 128;
  g.NL = alpha + 1;
  g.SB = ((g.NL * g.LS + 15) / 16) * 16;
  g.n_strips = std::max(1, (m + G * R - 1) / (G * R));
  return g;
}

// One (G, R) for all queries of a launch: minimise the modelled cell updates
// (row padding to whole strips, wavefront fill of G-1 columns per pair and
// strip, a per-step overhead amortised over R rows, a register-pressure
// penalty for the largest R).
// Small searches (few cells) are bound by their critical path -- one lane group
// sweeping the tallest query's strips over the longest short pair -- rather than by
// throughput.  Per wavefront step a lane spends about 18.4 cycles per row plus ~99
// of shuffles / loads (fit on config 1: G,R = 4,24 / 8,24 / 16,16 / 16,8 / 32,8 /
// 32,12 measured 1.11 / 0.60 / 0.39 / 0.45 / 0.26 / 0.38 ms, model within 12 %).
constexpr double SMALL_SEARCH_CELLS = 2e10;   // below this, minimise max(throughput, critical path)
constexpr double SMALL_LATENCY_CELLS = 1e9;   // below this, 32-lane groups get their own 32-thread CTAs
constexpr double CELLS_PER_CYCLE = 3500.0;    // whole-GPU throughput of the short-pair mode (config 3)

static void choose_geom(const sw_handle_s* h, const std::vector<std::pair<int, int>>& slots, double Lavg, int& G,
                        int& R, double Lmax = 0.0, double real_cells = 1e300, bool nib = false) {
  if (h->opt_G > 0 && h->opt_R > 0) {
    G = int(h->opt_G);
    R = int(h->opt_R);
    return;
  }
  static const int Gs[] = {4, 8, 16, 32};
  static const int Rs[] = {8, 12, 16, 20, 24, 28, 32};
  double best = 1e300;
  G = 4;
  R = 24;
  bool first = true;
  for (int g : Gs) {
    for (int r : Rs) {
      if (nib && !short_config_supported(slots.empty() ? 0 : slots[0].second, g, r, true)) continue;
      // per-step overhead amortised over r rows; a lane of one sub-lane (r % 8 != 0)
      // has half the ILP.  The single-query kernel spills above 24 rows; the
      // query-pair kernel (its own register budget) does not lose at 32 (C3 A/B:
      // (4,32) 7,034 vs (4,24) 6,902 vs (4,20) 6,496 GCUPS, profiles/r02_ab_geometry.txt).
      const bool qp = !slots.empty() && slots[0].second == 1;
      const double per_cell = 1.0 + 7.0 / (5.5 * r) + (r % 8 ? 0.06 : 0.0) + (!qp && r > 24 ? 0.06 : 0.0);
      double cost = 0;
      for (auto [m, mode] : slots) {
        const int strips = std::max(1, (m + g * r - 1) / (g * r));
        const double rows = double(strips) * g * r;
        // mode 1 (query pair) sweeps every DB sequence once for two queries, without the PRMT
        const double cols = mode == 1 ? 2.0 * (Lavg + g) * (5.5 / 6.5) : (Lavg + g);
        cost += rows * cols * per_cell * (strips > 1 ? 1.02 : 1.0);
        // single-query mode: each extra strip pass also costs ~6.7 cell-equivalents per
        // column (boundary-row round trip + pass setup; fit on config 2, where 3 passes
        // of G = 8 beat 6 passes of G = 4 by 1.9 % at equal row padding)
        if (mode == 0 && strips > 1) cost += 6.7 * double(strips) * Lavg;
      }
      if (real_cells < SMALL_SEARCH_CELLS && Lmax > 0) {  // in cycles: max(throughput, critical path)
        int mmax = 0;
        for (auto [m, mode] : slots) mmax = std::max(mmax, m);
        const int strips = std::max(1, (mmax + g * r - 1) / (g * r));
        const int V = (r % 8 == 0) ? 2 : 1;
        const double cp = double(strips) * (Lmax + double(g * V)) * (18.4 * r + 99.0);
        cost = std::max(cost / CELLS_PER_CYCLE, cp);
      }
      if (cost < best || first) { best = cost; G = g; R = r; first = false; }
    }
  }
}

// ----------------------------------------------------------------------------
extern "C" {

int32_t sw_init(int32_t device, uint32_t flags, sw_handle_t* out) {
  if (!out) return set_err(nullptr, SW_EINVAL, "sw_init: out is NULL");
  *out = nullptr;
  sw_handle_s* h = nullptr;
  int32_t rc = guarded(nullptr, [&] {
    int n = 0;
    SW_CK(cudaGetDeviceCount(&n));
    if (device < 0 || device >= n) fail(SW_EINVAL, "sw_init: bad device index");
    SW_CK(cudaSetDevice(device));
    h = new sw_handle_s();
    h->device = device;
    h->flags = flags;
    SW_CK(cudaDeviceGetAttribute(&h->sms, cudaDevAttrMultiProcessorCount, device));
  });
  if (rc != SW_OK) {
    delete h;
    return rc;
  }
  *out = h;
  return SW_OK;
}

int32_t sw_set_option(sw_handle_t h, const char* key, int64_t value) {
  if (!h || !key) return set_err(h, SW_EINVAL, "sw_set_option: NULL argument");
  std::string k(key);
  if (k == "overflow_threshold") h->opt_thr = value;
  else if (k == "force_G") {
    if (value != 0 && value != 4 && value != 8 && value != 16 && value != 32)
      return set_err(h, SW_EINVAL, "force_G must be 0, 4, 8, 16 or 32");
    h->opt_G = value;
  } else if (k == "force_R") {
    if (value != 0 && (value < 8 || value > 32 || value % 4))
      return set_err(h, SW_EINVAL, "force_R must be 0 or a multiple of 4 in [8, 32]");
    h->opt_R = value;
  } else if (k == "t_long") {
    if (value < 0) return set_err(h, SW_EINVAL, "t_long must be >= 0");
    h->opt_t_long = value;
  } else if (k == "align_workspace_mb") {
    if (value < 1) return set_err(h, SW_EINVAL, "sw_set_option: align_workspace_mb must be >= 1");
    h->opt_align_ws_mb = value;
  } else if (k == "pack_queries") {
    h->opt_pack_queries = value;
  } else if (k == "bank_copy") {
    h->opt_bank_copy = value;
  } else if (k == "bank_skew") {
    h->opt_bank_skew = value;
  } else if (k == "crit_min_steps") {
    if (value < 1) return set_err(h, SW_EINVAL, "crit_min_steps must be >= 1");
    h->opt_crit_min = value;
  } else if (k == "crit_pct") {
    if (value < 1) return set_err(h, SW_EINVAL, "crit_pct must be >= 1");
    h->opt_crit_pct = value;
  } else if (k == "rescore_rows") {
    if (value != 0 && value != 4 && value != 8) return set_err(h, SW_EINVAL, "rescore_rows must be 0, 4 or 8");
    h->opt_rescore_rows = value;
  } else if (k == "small_ctas") {
    h->opt_small_ctas = value;
  } else if (k == "nibble") {
    h->opt_nibble = value;
  } else if (k == "const_gaps") {
    h->opt_const_gaps = value;
  } else if (k == "query_pairs") {
    h->opt_query_pairs = value;
  } else if (k == "timing_accumulate") {
    h->timing_accumulate = value != 0;  // keep kernel events across searches until "timing_reset"
    h->n_events_used = 0;
  } else if (k == "timing_reset") {
    h->n_events_used = 0;
  } else if (k == "timing") {
    if (value) h->flags |= SW_FLAG_TIMING; else h->flags &= ~uint32_t(SW_FLAG_TIMING);
  } else
    return set_err(h, SW_EINVAL, "sw_set_option: unknown key " + k);
  return SW_OK;
}

int32_t sw_load_db(sw_handle_t h, const uint8_t* codes, const int64_t* offsets, int64_t n_seqs,
                   int32_t alphabet_size, void* cuda_stream, sw_db_t* out) {
  if (!h) return set_err(nullptr, SW_EINVAL, "sw_load_db: handle is NULL");
  if (!out) return set_err(h, SW_EINVAL, "sw_load_db: out is NULL");
  *out = nullptr;
  sw_db_s* db = nullptr;
  int32_t rc = guarded(h, [&] {
    SW_CK(cudaSetDevice(h->device));
    cudaStream_t st = reinterpret_cast<cudaStream_t>(cuda_stream);
    db = new sw_db_s();
    db->h = h;
    db->n_seqs = n_seqs;
    db->out_n = n_seqs;
    db->alpha = alphabet_size;
    Packed P;
    try {
      // nucleotide-sized alphabets (<= 15 codes + PAD) get the 4-bit stream
      pack_db(codes, offsets, n_seqs, alphabet_size, h->opt_t_long >= 0 ? h->opt_t_long : T_LONG, P,
              h->opt_nibble != 0 && alphabet_size <= 15);
    } catch (const std::invalid_argument& e) {
      fail(SW_EINVAL, std::string("sw_load_db: ") + e.what());
    }
    // strip progress counters encode (strip << 20) + column (kernels.cu): columns < 2^20
    if (P.max_len > (int64_t(1) << 20) - 128)
      fail(SW_EUNSUPPORTED, "sw_load_db: a sequence is longer than 2^20 - 128 residues");
    db->n_res = P.n_res;
    db->max_len = P.max_len;
    db->n_long = P.n_long;
    db->nib = P.nib;
    db->pairs = std::move(P.pairs);
    db->seq_len = std::move(P.seq_len);
    db->sorted_lens = std::move(P.sorted_lens);
    const size_t np = db->pairs.size();
    for (size_t p = 0; p < np; ++p) {
      const PairRec& r = db->pairs[p];
      if (int(p) < db->n_long) {
        db->sum_long_len += r.len;
        db->max_long = std::max(db->max_long, r.len);
      } else {
        db->sum_short_len += r.len;
        db->max_short = std::max(db->max_short, r.len);
        db->short_res += double(db->seq_len[size_t(r.id0)]) + (r.id1 >= 0 ? double(db->seq_len[size_t(r.id1)]) : 0.0);
      }
    }
    std::vector<uint16_t>& stream = P.stream;
    {  // prefix sums over the pairs (longest first): padded columns, real residues
      db->len_prefix.assign(np + 1, 0);
      db->res_prefix.assign(np + 1, 0.0);
      for (size_t p = 0; p < np; ++p) {
        const PairRec& r = db->pairs[p];
        db->len_prefix[p + 1] = db->len_prefix[p] + r.len;
        db->res_prefix[p + 1] = db->res_prefix[p] + double(db->seq_len[size_t(r.id0)]) +
                                (r.id1 >= 0 ? double(db->seq_len[size_t(r.id1)]) : 0.0);
      }
    }
    SW_CK(db->stream.ensure(stream.size() * sizeof(uint16_t)));
    SW_CK(db->dpairs.ensure(std::max<size_t>(np, 1) * sizeof(PairRec)));
    SW_CK(cudaMemcpyAsync(db->stream.p, stream.data(), stream.size() * sizeof(uint16_t), cudaMemcpyHostToDevice, st));
    if (np)
      SW_CK(cudaMemcpyAsync(db->dpairs.p, db->pairs.data(), np * sizeof(PairRec), cudaMemcpyHostToDevice, st));
    SW_CK(cudaStreamSynchronize(st));
  });
  if (rc != SW_OK) {
    delete db;
    return rc;
  }
  h->dbs.push_back(db);
  *out = db;
  return SW_OK;
}

int32_t sw_load_db_mapped(sw_handle_t h, const uint8_t* codes, const int64_t* offsets, int64_t n_seqs,
                          int32_t alphabet_size, const int64_t* out_index, int64_t out_n, void* cuda_stream,
                          sw_db_t* out) {
  if (!h) return set_err(nullptr, SW_EINVAL, "sw_load_db_mapped: handle is NULL");
  if (!out) return set_err(h, SW_EINVAL, "sw_load_db_mapped: out is NULL");
  if (n_seqs > 0 && !out_index) return set_err(h, SW_EINVAL, "sw_load_db_mapped: out_index is NULL");
  if (out_n < n_seqs) return set_err(h, SW_EINVAL, "sw_load_db_mapped: out_n < n_seqs");
  {  // distinct columns in [0, out_n)
    std::vector<uint8_t> seen(size_t(std::max<int64_t>(out_n, 1)), 0);
    for (int64_t d = 0; d < n_seqs; ++d) {
      const int64_t x = out_index[d];
      if (x < 0 || x >= out_n || seen[size_t(x)]) return set_err(h, SW_EINVAL, "sw_load_db_mapped: out_index not distinct in [0, out_n)");
      seen[size_t(x)] = 1;
    }
  }
  int32_t rc = sw_load_db(h, codes, offsets, n_seqs, alphabet_size, cuda_stream, out);
  if (rc != SW_OK) return rc;
  sw_db_s* db = *out;
  rc = guarded(h, [&] {
    cudaStream_t st = reinterpret_cast<cudaStream_t>(cuda_stream);
    // device pair table with output columns instead of caller indices (the host copy keeps them)
    std::vector<PairRec> dp(db->pairs);
    for (auto& r : dp) {
      r.id0 = int32_t(out_index[r.id0]);
      if (r.id1 >= 0) r.id1 = int32_t(out_index[r.id1]);
    }
    if (out_n > (int64_t(1) << 31) - 1) fail(SW_EUNSUPPORTED, "sw_load_db_mapped: out_n >= 2^31");
    if (!dp.empty())
      SW_CK(cudaMemcpyAsync(db->dpairs.p, dp.data(), dp.size() * sizeof(PairRec), cudaMemcpyHostToDevice, st));
    db->n_cols = n_seqs;
    if (n_seqs > 0) {
      SW_CK(db->dcols.ensure(size_t(n_seqs) * sizeof(int64_t)));
      SW_CK(cudaMemcpyAsync(db->dcols.p, out_index, size_t(n_seqs) * sizeof(int64_t), cudaMemcpyHostToDevice, st));
    }
    db->out_n = out_n;
    db->mapped = true;
    SW_CK(cudaStreamSynchronize(st));
  });
  if (rc != SW_OK) {
    sw_free_db(db);
    *out = nullptr;
  }
  return rc;
}

int32_t sw_db_info(sw_db_t db, sw_db_info_t* out) {
  if (!db || !out) return set_err(nullptr, SW_EINVAL, "sw_db_info: NULL argument");
  out->n_seqs = db->n_seqs;
  out->n_residues = db->n_res;
  out->n_pairs = int64_t(db->pairs.size());
  out->n_long_pairs = db->n_long;
  out->max_len = db->max_len;
  out->alphabet_size = db->alpha;
  out->device = db->h ? db->h->device : -1;
  return SW_OK;
}

static std::pair<cudaEvent_t, cudaEvent_t>* next_event_pair(sw_handle_s* h) {
  if (h->n_events_used == h->events.size()) {
    cudaEvent_t a, b;
    if (cudaEventCreate(&a) != cudaSuccess) return nullptr;
    if (cudaEventCreate(&b) != cudaSuccess) { cudaEventDestroy(a); return nullptr; }
    h->events.push_back({a, b});
    h->event_kind.push_back(0);
  }
  return &h->events[h->n_events_used++];
}

// The scoring launches of one search: profiles of every query, then the
// long-pair (intra-task) kernel (concurrently, when short pairs are scored too)
// and one persistent short-pair kernel per mode present (query pairs, single query).
struct LaunchCtx {
  sw_handle_s* h;
  sw_db_s* db;
  cudaStream_t st;
  int32_t* dscores;      // [nq][N]
  int32_t thr;
  OvfRec* ovf;
  int* ovf_count;
  int64_t ovf_cap;
  uint32_t nGe, nGsGe;
  bool timing;
};

struct LaunchOut {
  double cells_computed = 0, cells_short = 0;
  int launches = 0;
};

static void record_begin(sw_handle_s* h, bool timing, int kind, cudaStream_t st, std::pair<cudaEvent_t, cudaEvent_t>*& ev) {
  ev = timing ? next_event_pair(h) : nullptr;
  if (ev) {
    h->event_kind[h->n_events_used - 1] = kind;
    SW_CK(cudaEventRecord(ev->first, st));
  }
}

static void launch_all(LaunchCtx& c, const std::vector<int64_t>& qlen, const std::vector<int64_t>& qoff0,
                       LaunchOut& out) {
  sw_handle_s* h = c.h;
  sw_db_s* db = c.db;
  const int alpha = db->alpha;
  const int np = int(db->pairs.size());
  std::vector<int> order;
  for (int i = 0; i < int(qlen.size()); ++i)
    if (qlen[size_t(i)] > 0) order.push_back(i);
  if (order.empty() || np == 0) return;
  std::stable_sort(order.begin(), order.end(), [&](int x, int y) { return qlen[size_t(x)] > qlen[size_t(y)]; });
  std::vector<int> ms;
  for (int i : order) ms.push_back(int(qlen[size_t(i)]));
  const bool pairs_on = h->opt_query_pairs != 0;
  // geometry per mode from the plain neighbour pairing (mode 1: two queries per register)
  std::vector<std::pair<int, int>> m1, m0;
  for (size_t k = 0; k < order.size();) {
    if (pairs_on && k + 1 < order.size()) { m1.push_back({ms[k], 1}); k += 2; }
    else { m0.push_back({ms[k], 0}); k += 1; }
  }
  const int nshort_db = np - db->n_long;  // (only for the geometry cost model)
  const double Lavg = nshort_db > 0 ? db->sum_short_len / nshort_db : 1.0;
  double qsum = 0;
  for (int m : ms) qsum += m;
  int G1 = 4, R1 = 24, G0 = 4, R0 = 24;
  const bool nib = db->nib != 0;
  if (!m1.empty()) choose_geom(h, m1, Lavg, G1, R1, double(db->max_short), qsum * double(db->n_res), nib);
  if (!m0.empty()) choose_geom(h, m0, Lavg, G0, R0, double(db->max_short), qsum * double(db->n_res), nib);
  if (!m1.empty() && !short_config_supported(1, G1, R1, nib))
    fail(SW_EUNSUPPORTED, "no query-pair kernel for this geometry" + std::string(nib ? " (4-bit stream)" : ""));
  if (!m0.empty() && !short_config_supported(0, G0, R0, nib))
    fail(SW_EUNSUPPORTED, "no single-query kernel for this geometry" + std::string(nib ? " (4-bit stream)" : ""));
  // Latency-bound single-query searches (C1-sized) with 32-lane groups run one
  // lane group per 32-thread CTA: the groups then spread over all SMs instead of
  // eight per CTA sharing one SM's ALU pipe, which shortens the critical path.
  const bool small_ctas = !m0.empty() && G0 == 32 && qsum * double(db->n_res) < SMALL_LATENCY_CELLS &&
                          h->opt_small_ctas != 0 && short_config_supported(0, G0, R0, nib, 32);
  int NT0 = SCORE_NT;
  const int NT1 = SCORE_NT, NG1 = NT1 / G1, W = LONG_W;
  int NG0 = NT0 / G0;
  auto pairs_longer_than = [&](int64_t Lc) {  // pairs are sorted longest first
    int lo = 0, hi = np;
    while (lo < hi) { const int mid = (lo + hi) / 2; if (db->pairs[size_t(mid)].len > Lc) lo = mid + 1; else hi = mid; }
    return lo;
  };
  // Short-pair slots.  Mode 1: half A (low) and half B (high) each hold a list of
  // queries laid end to end on strip boundaries; the slot runs max(strips A,
  // strips B) strips.  The longest unplaced query opens a slot as half A and half
  // B takes the subset of the remaining queries whose strips best fill it (subset
  // sum), so the shorter half carries further queries instead of PAD rows.  A
  // last odd query runs alone in mode 0 (two DB sequences per register).
  struct Slot { int mode; std::vector<int> A, B; int strips, nlong; };
  std::vector<Slot> slots;
  {
    auto nst1 = [&](int k) { return std::max(1, (ms[size_t(k)] + G1 * R1 - 1) / (G1 * R1)); };
    std::vector<int> rem;
    for (size_t k = 0; k < order.size(); ++k) rem.push_back(int(k));  // longest first
    while (pairs_on && rem.size() >= 2) {
      const int a0 = rem[0];
      rem.erase(rem.begin());
      const int target = nst1(a0);
      std::vector<int> B;
      if (h->opt_pack_queries && double(rem.size()) * target <= 4e6) {
        // best subset sum <= target over rem (0/1 knapsack on strip counts)
        const size_t n = rem.size();
        std::vector<std::vector<char>> take(n, std::vector<char>(size_t(target) + 1, 0));
        std::vector<int> bestv(size_t(target) + 1, -1);
        bestv[0] = 0;
        for (size_t i = 0; i < n; ++i) {
          const int w = nst1(rem[i]);
          for (int v = target; v >= w; --v)
            if (bestv[size_t(v - w)] >= 0 && bestv[size_t(v)] < 0) { bestv[size_t(v)] = 1; take[i][size_t(v)] = 1; }
        }
        int v = target;
        while (v > 0 && bestv[size_t(v)] < 0) --v;
        for (size_t i = n; i-- > 0 && v > 0;)
          if (take[i][size_t(v)]) { B.push_back(rem[i]); v -= nst1(rem[i]); }
      } else {
        B.push_back(rem[0]);  // plain neighbour pairing
      }
      std::sort(B.begin(), B.end());
      for (int b : B) rem.erase(std::find(rem.begin(), rem.end(), b));
      slots.push_back({1, {a0}, B, target, 0});
    }
    for (int k : rem) slots.push_back({0, {k}, {}, std::max(1, (ms[size_t(k)] + G0 * R0 - 1) / (G0 * R0)), 0});
  }
  // Long pairs per slot: a short item (one lane group, every strip of its slot in
  // turn) must not run much longer than an average lane group's share of the
  // whole search, or it becomes the tail.  Pairs [0, nlong) of a slot go to the
  // intra-task kernel.  Option "t_long" forces every pair longer than it there.
  double group_steps = 0, resident_groups = 0;  // wavefront steps of all short work if nothing went long
  for (auto& sl : slots) {
    const int VG = sl.mode == 1 ? G1 * (R1 % 8 == 0 ? 2 : 1) : G0 * (R0 % 8 == 0 ? 2 : 1);
    const double seqs = sl.mode == 1 ? 2.0 * np : double(np);
    const double cols = sl.mode == 1 ? 2.0 * db->len_prefix[size_t(np)] : double(db->len_prefix[size_t(np)]);
    group_steps += double(sl.strips) * (cols + seqs * VG);
  }
  resident_groups = 2.0 * h->sms * double(!m1.empty() ? NG1 : NG0);
  const double crit = std::max(double(h->opt_crit_min), 0.01 * double(h->opt_crit_pct) * group_steps / resident_groups);
  // Long-sequence databases (most residues in pairs longer than T_LONG, config 4)
  // are scored entirely by the intra-task kernel; otherwise the critical-path
  // rule alone decides.
  int nlong_opt = 0;
  if (h->opt_t_long >= 0) {
    nlong_opt = pairs_longer_than(h->opt_t_long);
  } else {
    const int nT = pairs_longer_than(T_LONG);
    if (double(db->len_prefix[size_t(nT)]) > 0.5 * double(db->len_prefix[size_t(np)])) nlong_opt = nT;
  }
  for (auto& sl : slots) sl.nlong = std::max(nlong_opt, pairs_longer_than(int64_t(crit / sl.strips)));
  std::vector<int> qnlong(order.size(), 0);
  for (auto& sl : slots) {
    for (int k : sl.A) qnlong[size_t(k)] = sl.nlong;
    for (int k : sl.B) qnlong[size_t(k)] = sl.nlong;
  }
  // single-query searches with long pairs run as ONE combined launch (long items
  // first, one pair per item); otherwise the long kernel packs short queries' pairs
  bool any_q2 = false, any_m0 = false, any_long = false;
  for (auto& sl : slots) {
    if (sl.nlong < np) (sl.mode == 1 ? any_q2 : any_m0) = true;
    if (sl.nlong > 0) any_long = true;
  }
  const bool combined = any_long && any_m0 && !any_q2;  // (vs the forked long kernel on C2: 20.7 vs 28.7 ms,
                                                        //  profiles/r02_ab_combined_forms.txt)
  const int LR = combined ? LONG_R_COMBINED : LONG_R;  // rows per lane of the long path
  // ---- profiles: long geometry per query (if it has long pairs); short geometry per slot
  const int LB2 = (((R1 / 4) | 1) * 16);
  // Query-pair profile rows are LDS.128 per lane: a quarter-warp phase holds two
  // G = 4 groups reading random letters.  With LS2 a multiple of 128 B and odd
  // groups reading a second copy shifted by 64 B, the two groups always hit
  // disjoint bank halves ({k*LB2} mod 128 and {k*LB2 + 64} mod 128 partition the
  // eight 16-byte slots when LB2 is an odd multiple of 16).
  const bool bank_copy = h->opt_bank_copy != 0;
  const int LS2 = bank_copy ? ((G1 * LB2 + 127) / 128) * 128 : G1 * LB2;
  const int SB2 = (((alpha + 1) * LS2 + 15) / 16) * 16;
  const int ncopy2 = bank_copy ? std::max(1, (128 / 16) / G1) : 1;
  const ProfGeom g0 = make_geom(G0, R0, 1, alpha, false, bank_copy);  // SB / LS / LB of the mode-0 profile
  size_t total = 0;
  std::vector<ProfGeom> gl;
  std::vector<size_t> off_l;
  for (size_t k = 0; k < order.size(); ++k) {
    gl.push_back(make_geom(32, LR, ms[k], alpha, /*long_mode=*/true));
    off_l.push_back(total);
    total += qnlong[k] > 0 ? size_t(gl.back().n_strips) * gl.back().SB : 0;
  }
  std::vector<size_t> off_s;
  for (auto& sl : slots) {
    off_s.push_back(total);
    if (sl.nlong < np) total += size_t(sl.strips) * (sl.mode == 1 ? SB2 : g0.SB);
  }
  SW_CK(h->prof.ensure(total + 16));
  uint8_t* prof = h->prof.as<uint8_t>();
  const int8_t* dmat = h->matrix.as<int8_t>();
  auto qptr = [&](int k) { return h->qcodes.as<uint8_t>() + qoff0[size_t(order[size_t(k)])]; };
  auto pair_len_sum = [&](int p0, int p1) {  // sum of padded pair lengths over [p0, p1)
    return double(db->len_prefix[size_t(p1)] - db->len_prefix[size_t(p0)]);
  };
  auto pair_res_sum = [&](int p0, int p1) { return db->res_prefix[size_t(p1)] - db->res_prefix[size_t(p0)]; };
  if (small_ctas && !combined) {  // (a combined launch needs whole CTAs for its long items)
    NT0 = 32;
    NG0 = NT0 / G0;
  }
  // ---- long work: one item per (query, long pair), or per `pack` pairs
  std::vector<LongQuery> ldesc;
  struct LItem { double cost; int q, it; };
  std::vector<LItem> litems;
  int64_t long_items = 0;
  int wrap_groups = 1;  // pair groups per CTA that need a round-wrap row
  int32_t max_long = 0;
  // Warps per pair GS and pairs per item P (P * GS <= W) per query, two plans:
  //  latency-first: GS = min(strips, W) (fewest rounds per pair), P = W / GS;
  //  efficiency-first: the fewest idle warp-rounds -- ns strips over GS warps take
  //    ceil(ns / GS) rounds and W - P * GS warps idle -- ties to the larger GS, at
  //    most max(ceil(ns / W), 5) rounds.
  // The plan with the smaller modelled makespan max(longest item, CTA-steps / CTA
  // slots) wins: few long pairs (C3's tall-query tail) want short items, a long-only
  // database (C4) wants busy warps.  The combined single-query launch keeps one
  // pair per item.
  std::vector<int> gs_lat(order.size(), 1), gs_eff(order.size(), 1);
  double span_lat = 0, span_eff = 0, work_lat = 0, work_eff = 0;
  for (size_t k = 0; k < order.size(); ++k) {
    const int nl = qnlong[k];
    if (nl <= 0) continue;
    const int ns = gl[k].n_strips;
    int ge = std::min(ns, W);
    double best_eff = -1;
    for (int g = std::min(ns, W); g >= 1; --g) {
      const int p = W / g, rr = (ns + g - 1) / g;
      if (rr > std::max((ns + W - 1) / W, 5)) continue;  // bounds the item's critical path
      const double eff = double(p) * ns / (double(W) * rr);
      if (eff > best_eff + 1e-9) { best_eff = eff; ge = g; }
    }
    gs_lat[k] = std::min(ns, W);
    gs_eff[k] = ge;
    for (int pl = 0; pl < 2; ++pl) {
      const int g = pl == 0 ? gs_lat[k] : gs_eff[k], P = W / g;
      const double rounds = double((ns + g - 1) / g), fill = double(g - 1) * (LINK_LAG_STEPS + 64);
      double& span = pl == 0 ? span_lat : span_eff;
      double& work = pl == 0 ? work_lat : work_eff;
      span = std::max(span, rounds * double(db->pairs[0].len + 64) + fill);
      for (int it = 0; it * P < nl; ++it) work += rounds * double(db->pairs[size_t(it * P)].len + 64) + fill;
    }
  }
  const double long_slots = double(h->sms);  // the long kernel holds one CTA per SM (LONG_R = 32)
  const bool plan_eff = !combined && std::max(span_eff, work_eff / long_slots) <
                                         std::max(span_lat, work_lat / long_slots);
  for (size_t k = 0; k < order.size(); ++k) {
    const int nl = qnlong[k];
    if (nl <= 0) continue;
    SW_CK(launch_build_profile(qptr(int(k)), ms[k], dmat, alpha, gl[k], prof + off_l[k], c.st));
    ++out.launches;
    LongQuery d{};
    d.prof_long = prof + off_l[k];
    d.scores = c.dscores + int64_t(order[k]) * db->out_n;
    d.n_strips = gl[k].n_strips;
    d.qidx = order[k];
    d.n_long = nl;
    const int ns = gl[k].n_strips;
    const int GS = plan_eff ? gs_eff[k] : gs_lat[k], P = combined ? 1 : W / GS;
    d.pack = P;
    d.gs = GS;
    if (ns > GS) wrap_groups = std::max(wrap_groups, P);
    // item cost: rounds x the item's longest pair (pairs are sorted longest first)
    const double rounds = double((ns + GS - 1) / GS);
    for (int it = 0; it * d.pack < nl; ++it)
      litems.push_back({rounds * double(db->pairs[size_t(it * d.pack)].len + 64), int(ldesc.size()), it});
    ldesc.push_back(d);
    long_items += (nl + d.pack - 1) / d.pack;
    max_long = std::max(max_long, db->pairs[0].len);
    out.cells_computed += 2.0 * (pair_len_sum(0, nl) + 64.0 * nl) * double(gl[k].n_strips) * 32 * LR;
  }
  // ---- short work: slots per mode
  std::vector<SlotDesc> sdesc(slots.size());
  size_t vq_total = 0, si_total = 0;
  for (auto& sl : slots)
    if (sl.mode == 1) { vq_total += 2 * size_t(sl.strips) * G1 * R1; si_total += size_t(sl.strips); }
  std::vector<StripInfo> sinfo(si_total);
  if (vq_total) {
    SW_CK(h->vq.ensure(vq_total));
    SW_CK(cudaMemsetAsync(h->vq.p, alpha, vq_total, c.st));
    SW_CK(h->sinfo.ensure(si_total * sizeof(StripInfo)));
  }
  size_t vq_off = 0, si_off = 0;
  int min_pb1 = np, min_pb0 = np, max_strips1 = 1, max_strips0 = 1;
  for (size_t j = 0; j < slots.size(); ++j) {
    const Slot& sl = slots[j];
    SlotDesc& d = sdesc[j];
    const int ns = np - sl.nlong;  // short pairs of this slot
    const int NGm = sl.mode == 1 ? NG1 : NG0;
    d.prof = prof + off_s[j];
    d.mode = sl.mode;
    d.n_strips = sl.strips;
    d.qidx0 = order[size_t(sl.A[0])];
    d.scores0 = c.dscores + int64_t(d.qidx0) * db->out_n;
    d.sinfo = nullptr;
    d.pair_begin = sl.nlong;
    d.n_items = ns > 0 ? (sl.mode == 1 ? (2 * ns + NGm - 1) / NGm : (ns + NGm - 1) / NGm) : 0;
    double rows_real = 0;
    for (int kq : sl.A) rows_real += ms[size_t(kq)];
    for (int kq : sl.B) rows_real += ms[size_t(kq)];
    if (sl.mode == 1) {
      const size_t GR = size_t(G1) * R1;
      uint8_t* vA = h->vq.as<uint8_t>() + vq_off;
      uint8_t* vB = vA + size_t(sl.strips) * GR;
      vq_off += 2 * size_t(sl.strips) * GR;
      StripInfo* si = sinfo.data() + si_off;
      d.sinfo = h->sinfo.as<StripInfo>() + si_off;
      si_off += size_t(sl.strips);
      for (int s0 = 0; s0 < sl.strips; ++s0) si[s0] = StripInfo{0xffffffffu, -1, -1, 0};
      for (int hf = 0; hf < 2; ++hf) {
        const std::vector<int>& L = hf == 0 ? sl.A : sl.B;
        uint8_t* dst = hf == 0 ? vA : vB;
        int st0 = 0;
        for (int kq : L) {
          const int n = std::max(1, (ms[size_t(kq)] + G1 * R1 - 1) / (G1 * R1));
          if (ms[size_t(kq)] > 0)
            SW_CK(cudaMemcpyAsync(dst + size_t(st0) * GR, qptr(kq), size_t(ms[size_t(kq)]), cudaMemcpyDeviceToDevice,
                                  c.st));
          if (st0 > 0) si[st0].keep &= hf == 0 ? 0xffff0000u : 0x0000ffffu;  // new query: zero boundary
          (hf == 0 ? si[st0 + n - 1].emit0 : si[st0 + n - 1].emit1) = order[size_t(kq)];
          st0 += n;
        }
      }
      if (ns > 0) {
        const int rows = sl.strips * G1 * R1;
        SW_CK(launch_build_profile_q2(vA, rows, vB, rows, dmat, alpha, G1, R1, LB2, LS2, d.n_strips, SB2,
                                      prof + off_s[j], c.st));
        ++out.launches;
        const double sumS = pair_len_sum(sl.nlong, np) + double(ns) * 2 * G1;
        out.cells_computed += 2.0 * (2.0 * sumS) * double(d.n_strips) * G1 * R1;  // every sequence, 2 queries
        min_pb1 = std::min(min_pb1, sl.nlong);
        max_strips1 = std::max(max_strips1, sl.strips);
      }
    } else if (ns > 0) {
      ProfGeom gq = g0;
      gq.n_strips = d.n_strips;
      SW_CK(launch_build_profile(qptr(sl.A[0]), ms[size_t(sl.A[0])], dmat, alpha, gq, prof + off_s[j], c.st));
      ++out.launches;
      const double sumS = pair_len_sum(sl.nlong, np) + double(ns) * 2 * G0;
      out.cells_computed += 2.0 * sumS * double(d.n_strips) * G0 * R0;
      min_pb0 = std::min(min_pb0, sl.nlong);
      max_strips0 = std::max(max_strips0, sl.strips);
    }
    if (ns > 0) out.cells_short += rows_real * pair_res_sum(sl.nlong, np);
  }
  // global order of the short items of each mode: k-way merge of the slots' chunk
  // lists (each already longest-first) by critical path = strips x first pair length
  std::vector<int2> imap;
  int n_items1 = 0, n_items0 = 0;
  for (int mode = 1; mode >= 0; --mode) {
    struct Head { double key; int slot, chunk; };
    auto cmp = [](const Head& x, const Head& y) { return x.key < y.key || (x.key == y.key && x.slot > y.slot); };
    std::vector<Head> heap;
    const int NGm = mode == 1 ? NG1 : NG0;
    auto key_of = [&](int j, int ch) {
      const SlotDesc& d = sdesc[size_t(j)];
      const int p = d.pair_begin + (d.mode == 1 ? (ch * NGm) / 2 : ch * NGm);
      return double(d.n_strips) * double(db->pairs[size_t(std::min(p, np - 1))].len + 8);
    };
    for (size_t j = 0; j < sdesc.size(); ++j)
      if (sdesc[j].mode == mode && sdesc[j].n_items > 0) heap.push_back({key_of(int(j), 0), int(j), 0});
    std::make_heap(heap.begin(), heap.end(), cmp);
    const size_t before = imap.size();
    while (!heap.empty()) {
      std::pop_heap(heap.begin(), heap.end(), cmp);
      Head hd = heap.back();
      heap.pop_back();
      imap.push_back(make_int2(hd.slot, hd.chunk));
      if (hd.chunk + 1 < sdesc[size_t(hd.slot)].n_items) {
        heap.push_back({key_of(hd.slot, hd.chunk + 1), hd.slot, hd.chunk + 1});
        std::push_heap(heap.begin(), heap.end(), cmp);
      }
    }
    (mode == 1 ? n_items1 : n_items0) = int(imap.size() - before);
  }
  if (long_items + int64_t(imap.size()) >= (int64_t(1) << 31)) fail(SW_EUNSUPPORTED, "too many work items");
  if (si_total)
    SW_CK(h->stage.copy(h->sinfo.p, sinfo.data(), si_total * sizeof(StripInfo), c.st));
  SW_CK(h->imap.ensure(std::max<size_t>(imap.size(), 1) * sizeof(int2)));
  if (!imap.empty())
    SW_CK(h->stage.copy(h->imap.p, imap.data(), imap.size() * sizeof(int2), c.st));
  // long items costliest first across all queries (so no big item starts late)
  std::stable_sort(litems.begin(), litems.end(), [](const LItem& x, const LItem& y) { return x.cost > y.cost; });
  std::vector<int2> lmap(litems.size());
  for (size_t i = 0; i < litems.size(); ++i) lmap[i] = make_int2(litems[i].q, litems[i].it);
  SW_CK(h->lmap.ensure(std::max<size_t>(lmap.size(), 1) * sizeof(int2)));
  if (!lmap.empty())
    SW_CK(h->stage.copy(h->lmap.p, lmap.data(), lmap.size() * sizeof(int2), c.st));
  SW_CK(h->qdesc.ensure(ldesc.size() * sizeof(LongQuery) + sdesc.size() * sizeof(SlotDesc) + 16));
  LongQuery* d_ldesc = h->qdesc.as<LongQuery>();
  SlotDesc* d_slots = reinterpret_cast<SlotDesc*>(h->qdesc.as<uint8_t>() + ldesc.size() * sizeof(LongQuery));
  if (!ldesc.empty())
    SW_CK(h->stage.copy(d_ldesc, ldesc.data(), ldesc.size() * sizeof(LongQuery), c.st));
  SW_CK(h->stage.copy(d_slots, sdesc.data(), sdesc.size() * sizeof(SlotDesc), c.st));
  SW_CK(h->counters.ensure(3 * sizeof(int)));
  SW_CK(cudaMemsetAsync(h->counters.p, 0, 3 * sizeof(int), c.st));
  int* counters = h->counters.as<int>();
  const uint32_t code_pad2 = uint32_t(alpha) | (uint32_t(alpha) << 8);

  // ---- launches.  Long items: the long-pair kernel.  With short work too it runs
  // concurrently on the handle's side stream (high priority), one CTA per SM (its
  // shared-memory request leaves no room for a short-pair CTA, so co-resident short
  // warps cannot stretch the longest pairs' critical path); the caller's stream
  // waits for it (fork / join events), so the search stays stream-ordered.
  const bool has_short = n_items1 > 0 || n_items0 > 0;
  const bool fork = long_items > 0 && has_short && !combined;
  LongArgs al{};
  int smem_long = 0;
  if (long_items > 0) {
    const ProfGeom& l0 = gl[size_t(std::find_if(qnlong.begin(), qnlong.end(), [](int v) { return v > 0; }) -
                                   qnlong.begin())];
    al.queries = d_ldesc;
    al.n_queries = int(ldesc.size());
    al.n_items = int(long_items);
    al.lmap = h->lmap.as<int2>();
    al.SBL = l0.SB; al.LSL = l0.LS; al.LBL = l0.LB;
    smem_long = (W - 1) * LONG_RING * int(sizeof(uint2)) + W * l0.SB;
    al.wcap = max_long + 64 + 8;
    al.stream = db->stream.as<uint16_t>();
    al.pairs = db->dpairs.as<PairRec>();
    al.work_counter = counters + (combined ? 0 : 2);
    al.thr = c.thr;
    al.ovf = c.ovf;
    al.ovf_count = c.ovf_count;
    al.ovf_cap = int(c.ovf_cap);
    al.code_pad2 = code_pad2;
    al.nGe = c.nGe;
    al.nGsGe = c.nGsGe;
  }
  if (long_items > 0 && !combined) {
    int smem = smem_long;
    // SM-exclusive when forked (see above); measured on C3 against co-resident long CTAs
    // (1 per SM), grids capped at 16 / 32 CTAs and a serial long-then-short order:
    // 1,142 vs 1,163 / 1,204 / 1,157 / 1,154 ms (profiles/r02_ab_long_placement.txt)
    if (fork) smem = std::max(smem, 200 * 1024);
    const int occ = long_max_ctas_per_sm(smem, nib);
    if (occ <= 0) fail(SW_ECUDA, "long-pair kernel does not fit on an SM");
    const int grid = int(std::max<int64_t>(1, std::min<int64_t>(long_items, int64_t(occ) * h->sms)));
    al.wrap_groups = wrap_groups;
    SW_CK(h->wrap.ensure(size_t(grid) * wrap_groups * al.wcap * sizeof(uint2)));
    al.wrap = h->wrap.as<uint2>();
    cudaStream_t lst = c.st;
    if (fork) {
      if (!h->side) {
        int lo_p = 0, hi_p = 0;
        SW_CK(cudaDeviceGetStreamPriorityRange(&lo_p, &hi_p));
        SW_CK(cudaStreamCreateWithPriority(&h->side, cudaStreamNonBlocking, hi_p));
        SW_CK(cudaEventCreateWithFlags(&h->ev_fork, cudaEventDisableTiming));
        SW_CK(cudaEventCreateWithFlags(&h->ev_join, cudaEventDisableTiming));
      }
      SW_CK(cudaEventRecord(h->ev_fork, c.st));
      SW_CK(cudaStreamWaitEvent(h->side, h->ev_fork, 0));
      lst = h->side;
    }
    std::pair<cudaEvent_t, cudaEvent_t>* ev = nullptr;
    record_begin(h, c.timing, 1, lst, ev);
    SW_CK(launch_long(grid, smem, al, lst, nib));
    if (ev) SW_CK(cudaEventRecord(ev->second, lst));
    if (fork) SW_CK(cudaEventRecord(h->ev_join, lst));
    ++out.launches;
    ++h->stats.n_score_launches;
  }
  for (int mode : {1, 0}) {
    const int n_short = mode == 1 ? n_items1 : n_items0;
    if (n_short == 0) continue;
    const int G = mode == 1 ? G1 : G0, R = mode == 1 ? R1 : R0;
    ShortArgs as{};
    as.slots = d_slots;
    as.n_slots = int(sdesc.size());
    as.n_items = n_short;
    as.item_map = h->imap.as<int2>() + (mode == 1 ? 0 : n_items1);
    int smem = 0;
    if (mode == 1) {
      as.SB = SB2; as.LS = LS2; as.LB = LB2;
      as.ncopy = ncopy2;
      as.cstride = SB2 + (ncopy2 > 1 ? 128 / ncopy2 : 0);
      as.cskew = 0;
      // two TMA-staged buffers (strip s and the prefetched strip s+1), 128-byte aligned
      smem = 2 * ((((ncopy2 - 1) * as.cstride + SB2) + 127) / 128 * 128);
    } else {
      const Mode0Copies mc0 = mode0_copies(G, R, g0.LB, g0.SB, bank_copy, h->opt_bank_skew != 0);
      as.SB = g0.SB; as.LS = g0.LS; as.LB = g0.LB;
      as.ncopy = mc0.ncopy;
      as.cstride = mc0.cstride;
      as.cskew = mc0.skew;
      smem = mc0.bytes;
    }
    const bool with_long = combined && mode == 0;
    if (with_long) smem = std::max(smem, smem_long);  // an item is short or long: the two uses share smem
    const bool cg = c.nGe == 0xfffefffeu && c.nGsGe == 0xfff4fff4u && h->opt_const_gaps != 0;
    const int nt = mode == 1 ? NT1 : NT0;
    const int occ = with_long ? combined_max_ctas_per_sm(G, R, smem, nib, cg)
                              : short_max_ctas_per_sm(mode, G, R, smem, cg, nib, nt);
    if (occ <= 0) fail(SW_ECUDA, "short-pair kernel does not fit on an SM");
    const int64_t items = int64_t(n_short) + (with_long ? long_items : 0);
    const int grid = int(std::max<int64_t>(1, std::min<int64_t>(items, int64_t(occ) * h->sms)));
    const int min_pb = mode == 1 ? min_pb1 : min_pb0, max_strips = mode == 1 ? max_strips1 : max_strips0;
    const int32_t max_short = min_pb < np ? db->pairs[size_t(min_pb)].len : 0;
    as.bcap = ((max_short + 4 * G + 8 + 4) + 3) / 4 * 4;  // wave width up to V*G sub-lanes + align pad
    DevBuf& bbuf = mode == 1 ? h->bbuf1 : h->bbuf0;
    const int NT = mode == 1 ? NT1 : NT0;
    if (max_strips > 1) SW_CK(bbuf.ensure(size_t(grid) * (NT / G) * as.bcap * sizeof(uint2)));
    as.bbuf = max_strips > 1 ? bbuf.as<uint2>() : nullptr;
    as.stream = db->stream.as<uint16_t>();
    as.pairs = db->dpairs.as<PairRec>();
    as.pair_end = np;
    as.work_counter = counters + mode;
    as.scores_all = c.dscores;
    as.n_seqs = db->out_n;
    as.thr = c.thr;
    as.ovf = c.ovf;
    as.ovf_count = c.ovf_count;
    as.ovf_cap = int(c.ovf_cap);
    as.code_pad2 = code_pad2;
    as.nGe = c.nGe;
    as.nGsGe = c.nGsGe;
    std::pair<cudaEvent_t, cudaEvent_t>* ev = nullptr;
    record_begin(h, c.timing, 0, c.st, ev);
    if (with_long) {
      al.wrap_groups = wrap_groups;
      SW_CK(h->wrap.ensure(size_t(grid) * wrap_groups * al.wcap * sizeof(uint2)));
      al.wrap = h->wrap.as<uint2>();
      SW_CK(launch_combined(G, R, grid, smem, as, al, c.st, nib, cg));
    } else {
      SW_CK(launch_short(mode, G, R, grid, smem, as, c.st, cg, nib, nt));
    }
    if (ev) SW_CK(cudaEventRecord(ev->second, c.st));
    ++out.launches;
    ++h->stats.n_score_launches;
    h->stats.last_G = G;
    h->stats.last_R = R;
  }
  if (fork) SW_CK(cudaStreamWaitEvent(c.st, h->ev_join, 0));
}

int32_t sw_search(sw_handle_t h, const uint8_t* q_codes, const int64_t* q_offsets, int32_t n_queries, sw_db_t db,
                  const int8_t* matrix, int32_t gap_open, int32_t gap_extend, int32_t* scores, void* cuda_stream) {
  if (!h) return set_err(nullptr, SW_EINVAL, "sw_search: handle is NULL");
  return guarded(h, [&] {
    if (!db) fail(SW_EINVAL, "sw_search: db is NULL");
    if (db->h != h) fail(SW_ESTATE, "sw_search: db belongs to another handle");
    if (n_queries < 0) fail(SW_EINVAL, "sw_search: n_queries < 0");
    if (n_queries > 0 && !q_offsets) fail(SW_EINVAL, "sw_search: q_offsets is NULL");
    if (!matrix) fail(SW_EINVAL, "sw_search: matrix is NULL");
    if (gap_open < 0 || gap_extend < 0) fail(SW_EINVAL, "sw_search: gap penalties must be >= 0");
    if (int64_t(gap_open) + gap_extend > 32767) fail(SW_EINVAL, "sw_search: gap_open + gap_extend > 32767");
    const int alpha = db->alpha;
    SW_CK(cudaSetDevice(h->device));
    cudaStream_t st = reinterpret_cast<cudaStream_t>(cuda_stream);
    if (h->done_valid && h->done_stream != st) SW_CK(cudaStreamWaitEvent(st, h->ev_done, 0));
    h->stats = sw_stats_t{};
    if (!h->timing_accumulate) h->n_events_used = 0;
    h->last_stream = st;
    h->search_timed = false;
    if (n_queries == 0 || db->n_seqs == 0) return;
    if (!scores) fail(SW_EINVAL, "sw_search: scores is NULL");
    // queries
    std::vector<int64_t> qlen(static_cast<size_t>(n_queries));
    int64_t qtot = 0;
    for (int i = 0; i < n_queries; ++i) {
      qlen[size_t(i)] = q_offsets[i + 1] - q_offsets[i];
      if (qlen[size_t(i)] < 0) fail(SW_EINVAL, "sw_search: q_offsets not non-decreasing");
      // strip progress counters encode (strip << 20) + column: strips of >= 256 rows, < 2^11 of them
      if (qlen[size_t(i)] > (int64_t(1) << 19)) fail(SW_EUNSUPPORTED, "sw_search: query longer than 2^19 residues");
      qtot += qlen[size_t(i)];
    }
    if (qtot > 0 && !q_codes) fail(SW_EINVAL, "sw_search: q_codes is NULL");
    const uint8_t* qbase = q_codes ? q_codes + q_offsets[0] : nullptr;
    for (int64_t i = 0; i < qtot; ++i)
      if (qbase[i] >= alpha) fail(SW_EINVAL, "sw_search: query code >= alphabet_size");
    int smax = -128;
    for (int i = 0; i < alpha * alpha; ++i) smax = std::max<int>(smax, matrix[i]);
    // int16 re-score threshold: flag if max >= 32767 - S_max
    int32_t thr = smax > 0 ? 32767 - smax : 32768;
    // a forced threshold may only be lower: above 32767 - S_max a wrapped int16
    // value could pass unflagged
    if (h->opt_thr > 0) thr = int32_t(std::min<int64_t>(h->opt_thr, thr));
    // output
    cudaPointerAttributes pa{};
    bool dev_scores = false;
    if (cudaPointerGetAttributes(&pa, scores) == cudaSuccess)
      dev_scores = (pa.type == cudaMemoryTypeDevice || pa.type == cudaMemoryTypeManaged);
    cudaGetLastError();
    const int64_t N = db->out_n;  // row stride of the output (n_seqs unless the DB is mapped)
    const size_t out_bytes = size_t(n_queries) * size_t(N) * sizeof(int32_t);
    int32_t* dscores = scores;
    if (db->mapped && !dev_scores)
      fail(SW_EINVAL, "sw_search: a DB loaded with sw_load_db_mapped needs device (or peer-mapped) scores");
    if (!dev_scores) {
      SW_CK(h->scores_tmp.ensure(out_bytes));
      dscores = h->scores_tmp.as<int32_t>();
    }
    const bool timing = (h->flags & SW_FLAG_TIMING) != 0;
    if (timing) {
      if (!h->ev_begin) { SW_CK(cudaEventCreate(&h->ev_begin)); SW_CK(cudaEventCreate(&h->ev_end)); }
      SW_CK(cudaEventRecord(h->ev_begin, st));
    }
    // upload queries, offsets rebased to 0
    std::vector<int64_t> qoff0(size_t(n_queries) + 1);
    for (int i = 0; i <= n_queries; ++i) qoff0[size_t(i)] = q_offsets[i] - q_offsets[0];
    SW_CK(h->qcodes.ensure(size_t(std::max<int64_t>(qtot, 1))));
    SW_CK(h->qoff.ensure(qoff0.size() * sizeof(int64_t)));
    SW_CK(h->matrix.ensure(size_t(alpha * alpha)));
    SW_CK(h->stage.begin());
    SW_CK(h->stage.copy(h->qcodes.p, qbase, size_t(qtot), st));
    SW_CK(h->stage.copy(h->qoff.p, qoff0.data(), qoff0.size() * sizeof(int64_t), st));
    SW_CK(h->stage.copy(h->matrix.p, matrix, size_t(alpha * alpha), st));
    int launches = 0;
    if (!db->mapped) {
      SW_CK(cudaMemsetAsync(dscores, 0, out_bytes, st));
    } else if (db->n_cols > 0) {  // only this DB's columns (other ranks / shards own the rest)
      SW_CK(launch_zero_columns(dscores, N, n_queries, db->dcols.as<int64_t>(), db->n_cols, st));
      ++launches;
    }
    // overflow list capacity: a pair can only be flagged if min(m, n) * S_max >= thr
    int64_t ovf_cap = 0;
    if (smax > 0) {
      const int64_t need = std::max<int64_t>(1, (int64_t(thr) + smax - 1) / smax);  // min length that can reach thr
      // sorted_lens is descending: count the DB sequences of length >= need
      const int64_t nd_ge = std::lower_bound(db->sorted_lens.begin(), db->sorted_lens.end(), need,
                                             [](int64_t v, int64_t x) { return v >= x; }) -
                            db->sorted_lens.begin();
      for (int i = 0; i < n_queries; ++i)
        if (qlen[size_t(i)] >= need) ovf_cap += nd_ge;
    }
    if (ovf_cap > (int64_t(1) << 28)) fail(SW_EUNSUPPORTED, "sw_search: overflow list bound too large");
    SW_CK(h->ovf.ensure(size_t(std::max<int64_t>(ovf_cap, 1)) * sizeof(OvfRec)));
    SW_CK(h->ovf_count.ensure(sizeof(int)));
    SW_CK(cudaMemsetAsync(h->ovf_count.p, 0, sizeof(int), st));
    const int32_t max_short = db->max_short, max_long = db->max_long;
    const uint32_t nGe16 = uint32_t(uint16_t(int16_t(-gap_extend)));
    const uint32_t nGsGe16 = uint32_t(uint16_t(int16_t(-(gap_open + gap_extend))));
    LaunchCtx lc{};
    lc.h = h;
    lc.db = db;
    lc.st = st;
    lc.dscores = dscores;
    lc.thr = thr;
    lc.ovf = h->ovf.as<OvfRec>();
    lc.ovf_count = h->ovf_count.as<int>();
    lc.ovf_cap = ovf_cap;
    lc.nGe = nGe16 | (nGe16 << 16);
    lc.nGsGe = nGsGe16 | (nGsGe16 << 16);
    lc.timing = timing;
    LaunchOut lo;
    const uint8_t* dq = h->qcodes.as<uint8_t>();
    launch_all(lc, qlen, qoff0, lo);
    launches += lo.launches;
    if (ovf_cap > 0) {
      // Exact int32 re-score of the flagged pairs, enqueued unconditionally: the
      // kernel reads the flagged count on the device and exits at once when it is
      // zero, so the host never waits for the scoring kernel (stream-ordered).
      const int32_t Lmax = std::max(max_short, max_long);
      int64_t mmax = 1;
      for (auto L : qlen) mmax = std::max(mmax, L);
      const bool r4_ok = mmax <= int64_t(2047) * 32 * 4;  // (strip << 20) counters: < 2^11 strips
      const int rrows = (h->opt_rescore_rows == 8 || !r4_ok) ? RESCORE_R : 4;
      const int rows_per_strip = 32 * rrows;
      const int nstrips = int((mmax + rows_per_strip - 1) / rows_per_strip);
      // one round of RESCORE_WARPS strips per CTA (every wait targets an earlier item)
      const int K = std::max(1, (nstrips + RESCORE_WARPS - 1) / RESCORE_WARPS);
      const int grid = int(std::max<int64_t>(1, std::min<int64_t>(ovf_cap * K, 2 * h->sms)));
      const int ne_slots = int(std::min<int64_t>(ovf_cap, 64));
      const int bcap = Lmax + 32 + 72;
      SW_CK(h->rbuf.ensure(size_t(grid) * RESCORE_WARPS * bcap * sizeof(int2)));
      SW_CK(h->rgrows.ensure(size_t(ne_slots) * K * bcap * sizeof(int2) + 16));
      const size_t nflag_b = size_t(ne_slots) * K * sizeof(unsigned long long);
      const size_t nint = 2 * size_t(ovf_cap) + 1;
      SW_CK(h->rflags.ensure(nflag_b + nint * sizeof(int)));
      SW_CK(cudaMemsetAsync(h->rflags.p, 0, nflag_b + nint * sizeof(int), st));
      int* fl = reinterpret_cast<int*>(h->rflags.as<uint8_t>() + nflag_b);
      RescoreArgs r{};
      r.qcodes = dq;
      r.qoff = h->qoff.as<int64_t>();
      r.stream = db->stream.as<uint16_t>();
      r.nib = db->nib;
      r.pairs = db->dpairs.as<PairRec>();
      r.matrix = h->matrix.as<int8_t>();
      r.alpha = alpha;
      r.ovf = h->ovf.as<OvfRec>();
      r.ovf_count = h->ovf_count.as<int>();
      r.ovf_cap = int(ovf_cap);
      r.K = K;
      r.ne_slots = ne_slots;
      r.gflags = h->rflags.as<unsigned long long>();
      r.acc = fl;
      r.done = r.acc + ovf_cap;
      r.work_counter = r.done + ovf_cap;
      r.bbuf = h->rbuf.as<int2>();
      r.grows = h->rgrows.as<int2>();
      r.bcap = bcap;
      r.scores = dscores;
      r.n_seqs = N;
      r.Gs = gap_open;
      r.Ge = gap_extend;
      SW_CK(launch_rescore(grid, r, st, rrows));
      ++launches;
    }
    if (timing) {
      SW_CK(cudaEventRecord(h->ev_end, st));
      h->search_timed = true;
    }
    if (!h->ev_done) SW_CK(cudaEventCreateWithFlags(&h->ev_done, cudaEventDisableTiming));
    SW_CK(cudaEventRecord(h->ev_done, st));
    h->done_stream = st;
    h->done_valid = true;
    if (!dev_scores) {
      SW_CK(cudaMemcpyAsync(scores, dscores, out_bytes, cudaMemcpyDeviceToHost, st));
      SW_CK(cudaStreamSynchronize(st));
    }
    double sq = 0;
    for (auto L : qlen) sq += double(L);
    h->stats.cells = sq * double(db->n_res);
    h->stats.cells_short = lo.cells_short;  // scored by the short-pair (inter-task) kernels
    h->stats.cells_computed = lo.cells_computed;
    h->stats.n_launches = launches;
  });
}

// ----------------------------------------------------------------------------
// sw_align: int32 wavefront with 4-bit traceback codes, then a
// per-pair walk (align.cu).  Pairs are batched so that the codes of a batch fit
// the workspace budget.
int32_t sw_align(sw_handle_t h, const uint8_t* q_codes, const int64_t* q_offsets, int32_t n_queries, sw_db_t db,
                 const int32_t* pairs, int32_t n_pairs, const int8_t* matrix, int32_t gap_open, int32_t gap_extend,
                 int32_t* out5, uint32_t* ops, const int64_t* ops_offsets, int32_t* n_ops, void* cuda_stream) {
  if (!h) return set_err(nullptr, SW_EINVAL, "sw_align: handle is NULL");
  return guarded(h, [&] {
    if (!db) fail(SW_EINVAL, "sw_align: db is NULL");
    if (db->h != h) fail(SW_ESTATE, "sw_align: db belongs to another handle");
    if (n_pairs < 0 || n_queries < 0) fail(SW_EINVAL, "sw_align: negative count");
    if (n_pairs == 0) return;
    if (!pairs || !out5 || !n_ops || !ops_offsets || !q_offsets || !matrix)
      fail(SW_EINVAL, "sw_align: NULL argument");
    if (gap_open < 0 || gap_extend < 0) fail(SW_EINVAL, "sw_align: gap penalties must be >= 0");
    if (int64_t(gap_open) + gap_extend > (int64_t(1) << 24)) fail(SW_EINVAL, "sw_align: gap penalties too large");
    const int alpha = db->alpha;
    SW_CK(cudaSetDevice(h->device));
    cudaStream_t st = reinterpret_cast<cudaStream_t>(cuda_stream);
    std::vector<int64_t> qlen(static_cast<size_t>(n_queries));
    int64_t qtot = 0;
    for (int i = 0; i < n_queries; ++i) {
      qlen[size_t(i)] = q_offsets[i + 1] - q_offsets[i];
      if (qlen[size_t(i)] < 0) fail(SW_EINVAL, "sw_align: q_offsets not non-decreasing");
      if (qlen[size_t(i)] > (int64_t(1) << 19)) fail(SW_EUNSUPPORTED, "sw_align: query longer than 2^19 residues");
      qtot += qlen[size_t(i)];
    }
    if (qtot > 0 && !q_codes) fail(SW_EINVAL, "sw_align: q_codes is NULL");
    const uint8_t* qbase = q_codes ? q_codes + q_offsets[0] : nullptr;
    for (int64_t i = 0; i < qtot; ++i)
      if (qbase[i] >= alpha) fail(SW_EINVAL, "sw_align: query code >= alphabet_size");
    if (db->seq_loc.empty()) {
      db->seq_loc.assign(size_t(db->n_seqs), -1);
      for (size_t p = 0; p < db->pairs.size(); ++p) {
        db->seq_loc[size_t(db->pairs[p].id0)] = int64_t(2 * p);
        if (db->pairs[p].id1 >= 0) db->seq_loc[size_t(db->pairs[p].id1)] = int64_t(2 * p + 1);
      }
    }
    // items (pairs with an empty side are answered on the host)
    std::vector<AlignItem> items;
    std::vector<int32_t> item_pair;  // caller index of each item
    std::vector<int64_t> words;      // trace words per item
    for (int32_t k = 0; k < n_pairs; ++k) {
      const int32_t q = pairs[2 * k], d = pairs[2 * k + 1];
      if (q < 0 || q >= n_queries) fail(SW_EINVAL, "sw_align: query index out of range");
      if (d < 0 || int64_t(d) >= db->n_seqs) fail(SW_EINVAL, "sw_align: DB index out of range");
      if (ops_offsets[k + 1] < ops_offsets[k]) fail(SW_EINVAL, "sw_align: ops_offsets not non-decreasing");
      const int64_t m = qlen[size_t(q)], n = db->seq_len[size_t(d)];
      n_ops[k] = 0;
      out5[5 * k] = 0;
      for (int c = 1; c < 5; ++c) out5[5 * k + c] = -1;
      if (m == 0 || n == 0) continue;
      if (n > (int64_t(1) << 20) - 64) fail(SW_EUNSUPPORTED, "sw_align: DB sequence longer than 2^20 - 64");
      if (!ops && ops_offsets[k + 1] > ops_offsets[k]) fail(SW_EINVAL, "sw_align: ops is NULL");
      AlignItem it{};
      it.q = q;
      it.pair = int32_t(db->seq_loc[size_t(d)] >> 1);
      it.half = int32_t(db->seq_loc[size_t(d)] & 1);
      it.n = int32_t(n);
      it.ops_cap = int32_t(std::min<int64_t>(ops_offsets[k + 1] - ops_offsets[k], m + n + 1));
      items.push_back(it);
      item_pair.push_back(k);
      words.push_back((m + 255) / 256 * (((n + 3) & ~int64_t(3)) + 32) * 32);
    }
    if (items.empty()) return;
    // device inputs
    SW_CK(h->a_qcodes.ensure(size_t(std::max<int64_t>(qtot, 1))));
    SW_CK(h->a_qoff.ensure(size_t(n_queries + 1) * sizeof(int64_t)));
    SW_CK(h->a_matrix.ensure(size_t(alpha * alpha)));
    std::vector<int64_t> qoff0(static_cast<size_t>(n_queries + 1));
    for (int i = 0; i <= n_queries; ++i) qoff0[size_t(i)] = q_offsets[i] - q_offsets[0];
    if (qtot) SW_CK(cudaMemcpyAsync(h->a_qcodes.p, qbase, size_t(qtot), cudaMemcpyHostToDevice, st));
    SW_CK(cudaMemcpyAsync(h->a_qoff.p, qoff0.data(), qoff0.size() * sizeof(int64_t), cudaMemcpyHostToDevice, st));
    SW_CK(cudaMemcpyAsync(h->a_matrix.p, matrix, size_t(alpha * alpha), cudaMemcpyHostToDevice, st));
    SW_CK(h->a_counter.ensure(2 * sizeof(int)));
    // single-strip pairs (query <= 256 rows: one warp each) first, then the taller ones
    {
      std::vector<size_t> ord(items.size());
      std::iota(ord.begin(), ord.end(), size_t(0));
      std::stable_partition(ord.begin(), ord.end(), [&](size_t x) { return qlen[size_t(items[x].q)] <= 32 * ALIGN_R; });
      std::vector<AlignItem> it2;
      std::vector<int32_t> ip2;
      std::vector<int64_t> w2;
      for (size_t x : ord) { it2.push_back(items[x]); ip2.push_back(item_pair[x]); w2.push_back(words[x]); }
      items.swap(it2);
      item_pair.swap(ip2);
      words.swap(w2);
    }
    const int64_t budget = h->opt_align_ws_mb * (int64_t(1) << 20) / 4;  // words
    std::vector<uint32_t> hops;
    std::vector<int32_t> hout;
    size_t b0 = 0;
    while (b0 < items.size()) {
      // batch [b0, b1): trace words within budget (at least one item)
      size_t b1 = b0;
      int64_t tw = 0, ow = 0;
      int bcap = 0;
      while (b1 < items.size() && (b1 == b0 || tw + words[b1] <= budget)) {
        items[b1].trace_off = tw;
        items[b1].ops_off = ow;
        tw += words[b1];
        ow += items[b1].ops_cap;
        bcap = std::max(bcap, ((items[b1].n + 3) & ~3) + 32 + 8);
        ++b1;
      }
      const int nb = int(b1 - b0);
      SW_CK(h->a_items.ensure(size_t(nb) * sizeof(AlignItem)));
      SW_CK(h->a_trace.ensure(size_t(tw) * sizeof(uint32_t)));
      SW_CK(h->a_best.ensure(size_t(nb) * sizeof(int4)));
      SW_CK(h->a_ops.ensure(size_t(std::max<int64_t>(ow, 1)) * sizeof(uint32_t)));
      SW_CK(h->a_out.ensure(size_t(nb) * 6 * sizeof(int32_t)));
      int grid = std::min(nb, h->sms * 4);
      const int64_t link_budget = int64_t(1) << 30;  // bytes of warp link rows (HBM is plentiful)
      const int64_t per_cta = int64_t(ALIGN_WARPS) * bcap * int64_t(sizeof(int2));
      grid = int(std::max<int64_t>(1, std::min<int64_t>(grid, std::max<int64_t>(h->sms, link_budget / per_cta))));
      SW_CK(h->a_links.ensure(size_t(grid) * size_t(per_cta)));
      SW_CK(cudaMemsetAsync(h->a_counter.p, 0, 2 * sizeof(int), st));
      int n_single = 0;
      for (size_t x = b0; x < b1; ++x) n_single += qlen[size_t(items[x].q)] <= 32 * ALIGN_R ? 1 : 0;
      // very tall pairs (> 48 strips, queries > 12k rows): K = strips / 8 CTAs, one round
      // of 8 strips per CTA, so a CTA only ever waits on CTAs of lower sub-item index
      // (already running): no circular wait.  Shorter pairs keep one CTA and pipeline
      // their rounds inside it (measured: splitting config-3 top hits made them 2.6x slower).
      std::vector<int2> submap;
      for (size_t x = b0 + size_t(n_single); x < b1; ++x) {
        const int64_t ns = (qlen[size_t(items[x].q)] + 32 * ALIGN_R - 1) / (32 * ALIGN_R);
        const int K = ns > 6 * ALIGN_WARPS ? int((ns + ALIGN_WARPS - 1) / ALIGN_WARPS) : 1;
        items[x].K = K;
        for (int c = 0; c < K; ++c) submap.push_back(make_int2(int(x - b0), c));
      }
      for (size_t x = b0; x < b0 + size_t(n_single); ++x) items[x].K = 1;
      const int n_sub = int(submap.size());
      SW_CK(h->a_submap.ensure(std::max<size_t>(submap.size(), 1) * sizeof(int2)));
      SW_CK(h->a_grows.ensure(std::max<size_t>(submap.size(), 1) * size_t(bcap) * sizeof(int2)));
      SW_CK(h->a_gflags.ensure(std::max<size_t>(submap.size(), 1) * sizeof(int)));
      SW_CK(h->a_partial.ensure(std::max<size_t>(submap.size(), 1) * sizeof(int4)));
      SW_CK(h->a_done.ensure(size_t(nb) * sizeof(int)));
      if (n_sub) {
        SW_CK(cudaMemcpyAsync(h->a_submap.p, submap.data(), submap.size() * sizeof(int2), cudaMemcpyHostToDevice, st));
        SW_CK(cudaMemsetAsync(h->a_gflags.p, 0, submap.size() * sizeof(int), st));
      }
      SW_CK(cudaMemsetAsync(h->a_done.p, 0, size_t(nb) * sizeof(int), st));
      SW_CK(cudaMemcpyAsync(h->a_items.p, items.data() + b0, size_t(nb) * sizeof(AlignItem), cudaMemcpyHostToDevice,
                            st));
      AlignArgs a{};
      a.qcodes = h->a_qcodes.as<uint8_t>();
      a.qoff = h->a_qoff.as<int64_t>();
      a.stream = db->stream.as<uint16_t>();
      a.nib = db->nib;
      a.pairs = db->dpairs.as<PairRec>();
      a.matrix = h->a_matrix.as<int8_t>();
      a.alpha = alpha;
      a.items = h->a_items.as<AlignItem>();
      a.n_items = nb;
      a.work_counter = h->a_counter.as<int>();
      a.links = h->a_links.as<int2>();
      a.bcap = bcap;
      a.trace = h->a_trace.as<uint32_t>();
      a.best = h->a_best.as<int4>();
      a.ops = h->a_ops.as<uint32_t>();
      a.out = h->a_out.as<int32_t>();
      a.Gs = gap_open;
      a.Ge = gap_extend;
      a.submap = h->a_submap.as<int2>();
      a.n_sub = n_sub;
      a.grows = h->a_grows.as<int2>();
      a.gflags = h->a_gflags.as<int>();
      a.partial = h->a_partial.as<int4>();
      a.done = h->a_done.as<int>();
      SW_CK(launch_align(grid, n_single, a, h->a_counter.as<int>(), st));
      hout.resize(size_t(nb) * 6);
      hops.resize(size_t(std::max<int64_t>(ow, 1)));
      SW_CK(cudaMemcpyAsync(hout.data(), h->a_out.p, hout.size() * sizeof(int32_t), cudaMemcpyDeviceToHost, st));
      if (ow) SW_CK(cudaMemcpyAsync(hops.data(), h->a_ops.p, size_t(ow) * sizeof(uint32_t), cudaMemcpyDeviceToHost, st));
      SW_CK(cudaStreamSynchronize(st));
      for (int x = 0; x < nb; ++x) {
        const AlignItem& it = items[b0 + size_t(x)];
        const int32_t k = item_pair[b0 + size_t(x)];
        const int32_t* o = &hout[size_t(x) * 6];
        if (o[5] < 0 || o[5] > ops_offsets[k + 1] - ops_offsets[k])
          fail(SW_EINVAL, "sw_align: ops region of pair " + std::to_string(k) + " too small (needs " +
                              std::to_string(o[5] < 0 ? -o[5] : o[5]) + " entries)");
        for (int c = 0; c < 5; ++c) out5[5 * k + c] = o[c];
        n_ops[k] = o[5];
        if (o[5]) std::memcpy(ops + ops_offsets[k], &hops[size_t(it.ops_off)], size_t(o[5]) * sizeof(uint32_t));
      }
      b0 = b1;
    }
  });
}

// ----------------------------------------------------------------------------
// Merge of gathered score blocks.
int32_t sw_assembly_create(sw_handle_t h, const sw_block_t* blocks, int32_t n_blocks, const int32_t* rows,
                           int64_t n_rows, const int64_t* cols, int64_t n_cols, int32_t n_queries, int64_t N,
                           sw_assembly_t* out) {
  if (!h) return set_err(nullptr, SW_EINVAL, "sw_assembly_create: handle is NULL");
  if (!out) return set_err(h, SW_EINVAL, "sw_assembly_create: out is NULL");
  *out = nullptr;
  sw_assembly_s* a = nullptr;
  int32_t rc = guarded(h, [&] {
    if (n_blocks < 0 || n_rows < 0 || n_cols < 0 || n_queries < 0 || N < 0)
      fail(SW_EINVAL, "sw_assembly_create: negative size");
    if ((n_blocks > 0 && !blocks) || (n_rows > 0 && !rows) || (n_cols > 0 && !cols))
      fail(SW_EINVAL, "sw_assembly_create: NULL table");
    for (int64_t i = 0; i < n_rows; ++i)
      if (rows[i] < 0 || rows[i] >= n_queries) fail(SW_EINVAL, "sw_assembly_create: query index out of range");
    for (int64_t i = 0; i < n_cols; ++i)
      if (cols[i] < 0 || cols[i] >= N) fail(SW_EINVAL, "sw_assembly_create: column out of range");
    std::vector<AsmBlock> bk(static_cast<size_t>(n_blocks));
    std::vector<int64_t> prefix(size_t(n_blocks) + 1, 0);
    int64_t need = 0;
    for (int b = 0; b < n_blocks; ++b) {
      const sw_block_t& x = blocks[b];
      if (x.n_rows < 0 || x.n_cols < 0 || x.src_off < 0 || x.row_off < 0 || x.col_off < 0 ||
          x.row_off + x.n_rows > n_rows || x.col_off + x.n_cols > n_cols)
        fail(SW_EINVAL, "sw_assembly_create: block " + std::to_string(b) + " out of range");
      bk[size_t(b)] = AsmBlock{x.src_off, x.row_off, x.col_off, x.n_rows, x.n_cols};
      prefix[size_t(b) + 1] = prefix[size_t(b)] + x.n_rows * x.n_cols;
      need = std::max(need, x.src_off + x.n_rows * x.n_cols);
    }
    SW_CK(cudaSetDevice(h->device));
    a = new sw_assembly_s();
    a->h = h;
    a->n_blocks = n_blocks;
    a->total = prefix.back();
    a->src_need = need;
    a->n_queries = n_queries;
    a->N = N;
    SW_CK(a->blocks.ensure(std::max<size_t>(bk.size(), 1) * sizeof(AsmBlock)));
    SW_CK(a->prefix.ensure(prefix.size() * sizeof(int64_t)));
    SW_CK(a->rows.ensure(size_t(std::max<int64_t>(n_rows, 1)) * sizeof(int32_t)));
    SW_CK(a->cols.ensure(size_t(std::max<int64_t>(n_cols, 1)) * sizeof(int64_t)));
    if (n_blocks) SW_CK(cudaMemcpy(a->blocks.p, bk.data(), bk.size() * sizeof(AsmBlock), cudaMemcpyHostToDevice));
    SW_CK(cudaMemcpy(a->prefix.p, prefix.data(), prefix.size() * sizeof(int64_t), cudaMemcpyHostToDevice));
    if (n_rows) SW_CK(cudaMemcpy(a->rows.p, rows, size_t(n_rows) * sizeof(int32_t), cudaMemcpyHostToDevice));
    if (n_cols) SW_CK(cudaMemcpy(a->cols.p, cols, size_t(n_cols) * sizeof(int64_t), cudaMemcpyHostToDevice));
  });
  if (rc != SW_OK) {
    delete a;
    return rc;
  }
  h->assemblies.push_back(a);
  *out = a;
  return SW_OK;
}

int32_t sw_assemble(sw_assembly_t a, const int32_t* src, int64_t src_len, int32_t* out, void* cuda_stream) {
  if (!a || !a->h) return set_err(nullptr, SW_EINVAL, "sw_assemble: assembly is NULL");
  sw_handle_s* h = a->h;
  return guarded(h, [&] {
    if (src_len < a->src_need) fail(SW_EINVAL, "sw_assemble: src shorter than the blocks");
    if (a->total == 0) return;
    if (!src || !out) fail(SW_EINVAL, "sw_assemble: NULL buffer");
    SW_CK(cudaSetDevice(h->device));
    SW_CK(launch_assemble(src, a->blocks.as<AsmBlock>(), a->n_blocks, a->prefix.as<int64_t>(), a->total,
                          a->rows.as<int32_t>(), a->cols.as<int64_t>(), out, a->N, h->sms,
                          reinterpret_cast<cudaStream_t>(cuda_stream)));
  });
}

int32_t sw_assembly_free(sw_assembly_t a) {
  if (!a) return SW_OK;
  if (a->h) {
    cudaSetDevice(a->h->device);
    auto& v = a->h->assemblies;
    auto it = std::find(v.begin(), v.end(), a);
    if (it != v.end()) v.erase(it);
  }
  delete a;
  return SW_OK;
}

int32_t sw_last_stats(sw_handle_t h, sw_stats_t* out) {
  if (!h || !out) return set_err(h, SW_EINVAL, "sw_last_stats: NULL argument");
  return guarded(h, [&] {
    SW_CK(cudaSetDevice(h->device));
    SW_CK(cudaStreamSynchronize(h->last_stream));
    sw_stats_t s = h->stats;
    if (h->ovf_count.p) {
      int c = 0;
      SW_CK(cudaMemcpy(&c, h->ovf_count.p, sizeof(int), cudaMemcpyDeviceToHost));
      s.n_overflow = c;
    }
    double ms_s = 0, ms_l = 0;
    for (size_t i = 0; i < h->n_events_used; ++i) {
      float t = 0;
      SW_CK(cudaEventElapsedTime(&t, h->events[i].first, h->events[i].second));
      if (h->event_kind[i] == 0) ms_s += t; else ms_l += t;
    }
    s.short_ms = ms_s;
    s.long_ms = ms_l;
    s.search_ms = 0;
    if (h->search_timed) {
      float t = 0;
      SW_CK(cudaEventElapsedTime(&t, h->ev_begin, h->ev_end));
      s.search_ms = t;
    }
    s.timing_valid = h->n_events_used > 0 ? 1 : 0;
    *out = s;
  });
}

int32_t sw_free_db(sw_db_t db) {
  if (!db) return SW_OK;
  sw_handle_s* h = db->h;
  if (h) {
    cudaSetDevice(h->device);
    auto it = std::find(h->dbs.begin(), h->dbs.end(), db);
    if (it != h->dbs.end()) h->dbs.erase(it);
  }
  delete db;
  return SW_OK;
}

int32_t sw_free(sw_handle_t h) {
  if (!h) return SW_OK;
  cudaSetDevice(h->device);
  for (auto* db : h->dbs) {
    db->h = nullptr;
    delete db;
  }
  h->dbs.clear();
  for (auto* a : h->assemblies) delete a;
  h->assemblies.clear();
  for (auto& e : h->events) {
    cudaEventDestroy(e.first);
    cudaEventDestroy(e.second);
  }
  for (cudaEvent_t e : {h->ev_begin, h->ev_end, h->ev_fork, h->ev_join})
    if (e) cudaEventDestroy(e);
  if (h->side) cudaStreamDestroy(h->side);
  if (h->ev_done) cudaEventDestroy(h->ev_done);
  h->stage.release();
  delete h;
  return SW_OK;
}

const char* sw_last_error(sw_handle_t h) { return h ? h->err.c_str() : g_tls_err.c_str(); }

int32_t sw_encode_ascii(const char* s, int64_t n, uint8_t* out) {
  static const char* AL = "ARNDCQEGHILKMFPSTWYVBZX*";
  if (n < 0 || (n > 0 && (!s || !out))) return set_err(nullptr, SW_EINVAL, "sw_encode_ascii: bad argument");
  uint8_t lut[256];
  std::memset(lut, 22, sizeof(lut));  // X
  for (int k = 0; k < 24; ++k) {
    lut[uint8_t(AL[k])] = uint8_t(k);
    if (AL[k] >= 'A' && AL[k] <= 'Z') lut[uint8_t(AL[k] - 'A' + 'a')] = uint8_t(k);
  }
  lut[uint8_t('U')] = lut[uint8_t('u')] = 4;   // selenocysteine -> C
  lut[uint8_t('O')] = lut[uint8_t('o')] = 11;  // pyrrolysine -> K
  for (int64_t i = 0; i < n; ++i) out[i] = lut[uint8_t(s[i])];
  return SW_OK;
}

int32_t sw_search_cpu(const uint8_t* q_codes, const int64_t* q_offsets, int32_t n_queries, const uint8_t* db_codes,
                      const int64_t* db_offsets, int64_t n_seqs, int32_t alphabet_size, const int8_t* matrix,
                      int32_t gap_open, int32_t gap_extend, int32_t n_threads, int32_t* scores) {
  return guarded(nullptr, [&] {
    if (n_queries < 0 || n_seqs < 0) fail(SW_EINVAL, "sw_search_cpu: negative count");
    if (alphabet_size < 1 || alphabet_size > 32) fail(SW_EINVAL, "sw_search_cpu: alphabet_size must be 1..32");
    if (gap_open < 0 || gap_extend < 0) fail(SW_EINVAL, "sw_search_cpu: gap penalties must be >= 0");
    if (int64_t(gap_open) + gap_extend > 32767) fail(SW_EINVAL, "sw_search_cpu: gap_open + gap_extend > 32767");
    if (n_threads < 1) fail(SW_EINVAL, "sw_search_cpu: n_threads must be >= 1");
    if (n_queries == 0 || n_seqs == 0) return;
    if (!q_offsets || !db_offsets || !matrix || !scores) fail(SW_EINVAL, "sw_search_cpu: NULL argument");
    if (!__builtin_cpu_supports("avx2")) fail(SW_EUNSUPPORTED, "sw_search_cpu: the host CPU has no AVX2");
    auto check_codes = [&](const uint8_t* c, const int64_t* off, int64_t n, const char* what) {
      for (int64_t i = 0; i < n; ++i)
        if (off[i + 1] < off[i]) fail(SW_EINVAL, std::string("sw_search_cpu: ") + what + " offsets not non-decreasing");
      const int64_t tot = off[n] - off[0];
      if (tot > 0 && !c) fail(SW_EINVAL, std::string("sw_search_cpu: ") + what + " codes NULL");
      for (int64_t i = 0; i < tot; ++i)
        if (c[i] >= alphabet_size) fail(SW_EINVAL, std::string("sw_search_cpu: ") + what + " code >= alphabet_size");
    };
    check_codes(q_codes, q_offsets, n_queries, "query");
    check_codes(db_codes, db_offsets, n_seqs, "DB");
    swdual::cpu_search_avx2(q_codes, q_offsets, n_queries, db_codes, db_offsets, n_seqs, alphabet_size, matrix,
                            gap_open, gap_extend, n_threads, scores);
  });
}

int32_t sw_encode_nucleotide(const char* s, int64_t n, uint8_t* out) {
  if (n < 0 || (n > 0 && (!s || !out))) return set_err(nullptr, SW_EINVAL, "sw_encode_nucleotide: bad argument");
  uint8_t lut[256];
  std::memset(lut, 4, sizeof(lut));  // N and every other letter
  const char* AL = "ACGT";
  for (int k = 0; k < 4; ++k) {
    lut[uint8_t(AL[k])] = uint8_t(k);
    lut[uint8_t(AL[k] - 'A' + 'a')] = uint8_t(k);
  }
  lut[uint8_t('U')] = lut[uint8_t('u')] = 3;  // RNA uracil pairs like T
  for (int64_t i = 0; i < n; ++i) out[i] = lut[uint8_t(s[i])];
  return SW_OK;
}

}  // extern "C"
