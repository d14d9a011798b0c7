// Internal types shared by the host engine (engine.cpp) and the kernels (kernels.cu).
// Product code only: nothing here is shared with oracle/.
#pragma once
#include <cstdint>
#include <vector>
#include <cuda_runtime.h>

namespace swdual {

// One packed database "pair": two length-sorted neighbours interleaved column by
// column into 16-bit words (low byte = sequence id0, high byte = id1), padded to a
// multiple of 4 columns with the PAD code.  id1 = -1 for an odd leftover sequence.
struct PairRec {
  int64_t off;   // start, in 16-bit words, into the pair stream (multiple of 4)
  int32_t len;   // padded length (multiple of 4) = columns processed
  int32_t id0;   // caller's index of the low-half sequence
  int32_t id1;   // caller's index of the high-half sequence or -1
  int32_t pad_;
};

// Host-packed database (packer.cpp).  nib = 0: 16-bit pair columns (8-bit codes,
// protein); nib = 1 (alphabet <= 15, nucleotides): 8-bit pair
// columns of two 4-bit codes (low nibble id0, high nibble id1), stored as bytes
// in `stream`; pair p's column c is byte off + c.
struct Packed {
  std::vector<PairRec> pairs;        // sorted longest first
  std::vector<uint16_t> stream;      // interleaved pair columns (bytes when nib)
  int nib = 0;
  std::vector<int64_t> seq_len;      // caller order
  std::vector<int64_t> sorted_lens;  // non-empty lengths, descending
  int64_t n_res = 0, max_len = 0;
  int n_long = 0;                    // pairs [0, n_long) are longer than t_long
};
void pack_db(const uint8_t* codes, const int64_t* offsets, int64_t n_seqs, int alpha, int64_t t_long, Packed& P,
             bool nib = false);

// A pair whose int16 maximum reached the overflow threshold:
// re-scored exactly in int32.
struct OvfRec {
  int32_t q;     // query index within the search
  int32_t pair;  // pair index
  int32_t half;  // 0 = id0, 1 = id1
  int32_t pad_;
};

// Geometry of one query profile (int8, strip-major, lane-blocked; see kernels.cu).
struct ProfGeom {
  int G, R;        // lanes per group, rows per lane
  int LB;          // bytes per lane block (>= R, odd number of load units)
  int LS;          // bytes per letter = G * LB
  int NL;          // letters = alpha + 1 (PAD = alpha)
  int SB;          // bytes per strip (multiple of 16)
  int n_strips;    // ceil(m / (G*R))
  int UB;          // bytes per load unit (8 or 4)
  int il;          // 1: unit-interleaved [letter][unit][lane][UB] (long mode); 0: [letter][lane][LB]
};

// Rows per lane of the intra-task (long pair) geometry, G = 32 lanes; profile
// unit-interleaved ([letter][unit][lane][8 B]): dense and bank-conflict-free (the
// 16 lanes of an LDS.64 phase hit 16 distinct 8-byte slots whatever letters they read)
// Rows per lane of the long kernel (32: one CTA of 8 warps per SM, 25.6 KB of int8
// profile per warp; the per-step ring I/O, waits and code handling amortised over 32
// rows) and of the long path inside the combined single-query kernel (16: it shares
// the SM with a second CTA of short items).
constexpr int LONG_R = 32;
constexpr int LONG_R_COMBINED = 16;
constexpr int LONG_US = 32 * 8;     // bytes between a lane's consecutive 8-byte units in the long profile
constexpr int LONG_RING = 128;      // steps held by a shared-memory link ring between two warps of a CTA

// Long (intra-task) work of one query: pairs [0, n_long) of the DB are scored by
// the chained warps of one CTA each.
struct LongQuery {
  const uint8_t* prof_long;  // [n_strips][SBL] int8, 32 lanes x LONG_R rows per strip
  int32_t* scores;           // this query's row of scores[Q][N] (caller order)
  int n_strips;
  int qidx;
  int n_long;
  int pack;                  // pairs per item (P): the CTA's warps chain P pairs side by side
  int gs;                    // warps per pair (GS, P * GS <= W): a pair's strips go round-robin
                             // over its GS warps, ceil(n_strips / GS) rounds
};

struct LongArgs {
  const LongQuery* queries;  // [n_queries], processing order
  int n_queries;
  int n_items;               // long items of the launch
  const int2* lmap;          // item -> (query, item within the query), costliest first
  int SBL, LSL, LBL;         // long profile geometry
  uint2* wrap;               // [gridDim][wrap_groups][wcap]: the round-wrap link row of each pair
                             // group of a CTA (its last warp -> its first warp, next round)
  int wrap_groups;           // max pairs per item among queries of more strips than warps per pair
  int wcap;
  const uint16_t* stream;
  const PairRec* pairs;
  int* work_counter;
  int32_t thr;               // overflow threshold (int16 max >= thr -> re-score)
  OvfRec* ovf;
  int* ovf_count;
  int ovf_cap;
  uint32_t code_pad2;        // PAD | PAD << 8
  uint32_t nGe, nGsGe;       // packed s16x2 -Ge, -(Gs+Ge)
};

// Short-pair work of one "slot": a single query (mode 0: two DB sequences per
// s16x2 register, int8 profile) or a query PAIR (mode 1: two queries per
// register, one DB sequence per lane group, s16x2 profile).
// Mode-1 slots pack several queries per s16x2 half, each starting on a strip
// boundary (fills the shorter half of a query pair with
// further short queries instead of PAD rows).  Per strip of such a slot:
struct StripInfo {
  uint32_t keep;             // halves that continue the query of the previous strip (0x0000ffff: low
                             // half, 0xffff0000: high half); a new query starts from a zero boundary row
  int32_t emit0, emit1;      // query whose last strip this is, per half (-1: none)
  int32_t pad_;
};

struct SlotDesc {
  const StripInfo* sinfo;    // mode 1: [n_strips]
  const uint8_t* prof;       // mode 0: [n_strips][SB] int8; mode 1: [n_strips][SB] s16x2
  int32_t* scores0;          // mode 0: the query's scores row
  int n_strips;
  int mode;
  int qidx0;
  int n_items;               // short work items of this slot
  int pair_begin;            // short pairs of this slot: [pair_begin, pair_end)
  int pad_;
};

// One short-pair kernel launch (all slots of one mode).
struct ShortArgs {
  const SlotDesc* slots;
  int n_slots;
  int n_items;
  const int2* item_map;      // item -> (slot, chunk), longest critical path first
  int SB, LS, LB;            // strip profile geometry of this mode
  // Bank-spread copies of the strip profile in shared memory: lane group g reads
  // copy g % ncopy at ncopy-dependent offsets (copy_off), so the groups of one
  // shared-memory phase (random letters each) hit disjoint banks.
  int ncopy, cstride;
  uint32_t cskew;            // per-copy 4-byte skews (mode 0), 0 for the linear layout
  const uint16_t* stream;
  const PairRec* pairs;
  int pair_end;
  uint2* bbuf;               // boundary rows of multi-strip items, [gridDim][NG][bcap]
  int bcap;
  int* work_counter;
  int32_t* scores_all;       // [n_queries (caller order)][n_seqs]
  int64_t n_seqs;
  int32_t thr;
  OvfRec* ovf;
  int* ovf_count;
  int ovf_cap;
  uint32_t code_pad2;
  uint32_t nGe, nGsGe;
};

struct RescoreArgs {
  const uint8_t* qcodes;     // all queries, concatenated
  const int64_t* qoff;       // [nq+1]
  const uint16_t* stream;
  int nib;                   // 4-bit pair columns (bytes) instead of 16-bit
  const PairRec* pairs;
  const int8_t* matrix;      // alpha x alpha
  int alpha;
  const OvfRec* ovf;         // flagged pairs
  const int* ovf_count;      // device: flagged pairs written by the scoring kernel (read on the device,
  int ovf_cap;               //   so the host never waits for it); entries = min(*ovf_count, ovf_cap)
  int K;                     // CTAs per flagged pair (one round of RESCORE_WARPS strips each)
  int ne_slots;              // CTA-to-CTA row blocks: entry e uses block e % ne_slots
  int* work_counter;         // zeroed
  int2* bbuf;                // per-CTA warp link rows, [gridDim][RESCORE_WARPS][bcap]
  int2* grows;               // CTA-to-CTA rows, [ne_slots][K][bcap]
  unsigned long long* gflags;  // [ne_slots][K]: (entry + 1) << 32 | progress (generation-tagged), zeroed
  int* acc;                  // [ovf_cap] partial maxima, zeroed
  int* done;                 // [ovf_cap] finished CTAs per entry, zeroed
  int bcap;
  int32_t* scores;           // [nq][n_seqs]
  int64_t n_seqs;
  int32_t Gs, Ge;
};

// One gathered score block (sw_assemble): rows x cols int32 at src + src_off.
struct AsmBlock {
  int64_t src_off;   // elements
  int64_t row_off;   // into the rows table (query indices)
  int64_t col_off;   // into the cols table (DB columns)
  int64_t n_rows, n_cols;
};

// kernels.cu entry points (host side launchers); return cudaError_t
cudaError_t launch_build_profile(const uint8_t* q, int m, const int8_t* matrix, int alpha,
                                 const ProfGeom& g, uint8_t* prof, cudaStream_t st);
// query-pair profile: word = S[qa_i][a] (low 16) | S[qb_i][a] << 16, lane block LB2
cudaError_t launch_build_profile_q2(const uint8_t* qa, int ma, const uint8_t* qb, int mb, const int8_t* matrix,
                                    int alpha, int G, int R, int LB2, int LS2, int n_strips, int SB2, uint8_t* prof,
                                    cudaStream_t st);
// Short-pair kernels: mode 0 (single query) and mode 1 (query pairs), one (G, R)
// per launch.  Long-pair kernel: LONG_W chained warps per CTA.
constexpr int SCORE_NT = 256;       // threads per CTA of both
constexpr int LONG_W = SCORE_NT / 32;
// cg: the gaps are Gs = 10, Ge = 2 -- use the constant-gap instantiation when one exists;
// nib: the DB stream holds 4-bit codes (only the SW_NIB_CASES geometries exist)
// nt: threads per CTA (SCORE_NT, or 32 for latency-bound single-query searches at G = 32)
bool short_config_supported(int mode, int G, int R, bool nib = false, int nt = SCORE_NT);
int short_max_ctas_per_sm(int mode, int G, int R, int smem_bytes, bool cg = false, bool nib = false,
                          int nt = SCORE_NT);
cudaError_t launch_short(int mode, int G, int R, int grid, int smem_bytes, const ShortArgs& a, cudaStream_t st,
                         bool cg = false, bool nib = false, int nt = SCORE_NT);
int long_max_ctas_per_sm(int smem_bytes, bool nib = false);
cudaError_t launch_long(int grid, int smem_bytes, const LongArgs& a, cudaStream_t st, bool nib = false);
// single-query searches with long pairs: long items and mode-0 short items in one launch
int combined_max_ctas_per_sm(int G, int R, int smem_bytes, bool nib = false, bool cg = false);
cudaError_t launch_combined(int G, int R, int grid, int smem_bytes, const ShortArgs& as, const LongArgs& al,
                            cudaStream_t st, bool nib = false, bool cg = false);
// rows: rows per lane, RESCORE_R or 4 (only when every query has < 2^11 strips of 128 rows)
cudaError_t launch_rescore(int grid, const RescoreArgs& a, cudaStream_t st, int rows);
// scores[q * stride + cols[c]] = 0 for every query q < nq and column c < ncols
cudaError_t launch_zero_columns(int32_t* scores, int64_t stride, int nq, const int64_t* cols, int64_t ncols,
                                cudaStream_t st);
cudaError_t launch_assemble(const int32_t* src, const AsmBlock* blocks, int n_blocks, const int64_t* prefix,
                            int64_t total, const int32_t* rows, const int64_t* cols, int32_t* out, int64_t N,
                            int sms, cudaStream_t st);
constexpr int RESCORE_WARPS = 8;
constexpr int RESCORE_R = 8;  // rows per lane; 4 for searches whose queries all have < 2^11 strips of
                              // 128 rows (C4: 13.3 vs 14.9 ms, 16 rows 22 ms, profiles/r02_ab_rescore_rows.txt)


// Best local alignment of selected pairs (align.cu).  One item =
// one (query, DB sequence) pair; its traceback codes live at trace + trace_off:
// [strip][step t][lane] u32 words, 8 rows x 4 bits per word (see align.cu).
struct AlignItem {
  int64_t trace_off;         // u32 words
  int64_t ops_off;           // u32 run-length codes: this item's output region
  int32_t q;                 // query index (qoff)
  int32_t pair;              // packed pair holding the DB sequence
  int32_t half;              // 0 = low byte (id0), 1 = high byte (id1)
  int32_t n;                 // real DB sequence length
  int32_t ops_cap;           // capacity of the output region
  int32_t K;                 // CTAs the pair is split over (tall queries)
};

struct AlignArgs {
  const uint8_t* qcodes;     // all queries, concatenated
  const int64_t* qoff;       // [nq+1]
  const uint16_t* stream;
  int nib;                   // 4-bit pair columns (bytes) instead of 16-bit
  const PairRec* pairs;
  const int8_t* matrix;      // alpha x alpha
  int alpha;
  const AlignItem* items;    // this batch
  int n_items;               // items of the batch (traceback launch)
  int item_begin, n_launch;  // single-strip launch: items [item_begin, item_begin + n_launch)
  const int2* submap;        // tall-pair launch: sub-item -> (item, CTA c of K), a pair's K consecutive
  int n_sub;
  int2* grows;               // CTA-to-CTA rows, [n_sub][bcap]
  int* gflags;               // their progress counters, [n_sub], zeroed
  int4* partial;             // per sub-item best {v, j, i}
  int* done;                 // per item finished CTAs, zeroed
  int* work_counter;         // zeroed
  int2* links;               // per-CTA warp link rows, [gridDim][ALIGN_WARPS][bcap]
  int bcap;
  uint32_t* trace;           // traceback codes of the batch
  int4* best;                // per item: {score, end row i (1-based), end column j (1-based), 0}
  uint32_t* ops;             // run-length codes, per item at ops_off (written reversed, then flipped)
  int32_t* out;              // per item: {score, q_begin, q_end, d_begin, d_end, n_ops (< 0: region too small)}
  int32_t Gs, Ge;
};

// CPU-type PE (cpu_striped.cpp, AVX2): scores[q][d] for all pairs, host only.
void cpu_search_avx2(const uint8_t* qcodes, const int64_t* qoff, int32_t nq, const uint8_t* dcodes,
                     const int64_t* doff, int64_t n_seqs, int alpha, const int8_t* S, int32_t Gs, int32_t Ge,
                     int32_t n_threads, int32_t* scores);

constexpr int ALIGN_WARPS = 8;
constexpr int ALIGN_R = 8;   // rows per lane = codes per trace word
cudaError_t launch_align(int grid, int n_single, const AlignArgs& a, int* counters, cudaStream_t st);

}  // namespace swdual
