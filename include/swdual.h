/*
 * swdual.h -- C ABI of the B200-native SWDUAL hot path.
 *
 * Computes, for a set of queries and a database of sequences, the
 * Smith-Waterman local-alignment score with affine gaps (Gotoh) of every
 * (query, database sequence) pair -- the computation the SWDUAL scheduler of
 * Kedad-Sidhoum et al., ICPP 2014 distributes over CPUs and GPUs.
 * PAPER.md = /root/reference/PAPER.md; citations give line numbers there.
 *
 *   "compare a set q of m query sequences to a set d of n database
 *    sequences"                                         (L196-201, sec. II.C)
 *   H_ij = max(H_{i-1,j-1} + S_ij, E_ij, F_ij, 0)              (Eq. (2))
 *   E_ij = -Ge + max(E_{i,j-1}, H_{i,j-1} - Gs)                 (Eq. (3))
 *   F_ij = -Ge + max(F_{i-1,j}, H_{i-1,j} - Gs)                 (Eq. (4))
 *   first row and column of H are zero                           (L153-154)
 *   result = the maximal score, "the similarity"                  (L135-136)
 *
 * so a gap of k residues costs gap_open + k * gap_extend (Gs + k*Ge).
 *
 * Conventions for every entry point:
 *   - return int32 status: SW_OK (0) or a negative SW_E* code; no exception
 *     crosses the ABI; sw_last_error() describes the last failure of a handle.
 *   - "host" pointers are read/written by the CPU; "host or device" pointers
 *     may be either (cudaPointerGetAttributes decides); the caller owns all
 *     buffers it passes in and may free them when the call returns.
 *   - a handle is bound to one CUDA device and is not thread-safe: one call at
 *     a time per handle.
 *   - cuda_stream is a cudaStream_t (NULL = legacy default stream).
 */
#ifndef SWDUAL_H
#define SWDUAL_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct sw_handle_s* sw_handle_t; /* opaque; bound to one CUDA device   */
typedef struct sw_db_s* sw_db_t;         /* opaque; packed, device-resident DB  */

enum {
  SW_OK = 0,
  SW_EINVAL = -1,       /* bad argument (null pointer, code >= alphabet, ...) */
  SW_ENOMEM = -2,       /* device or host allocation failed                    */
  SW_ECUDA = -3,        /* a CUDA call failed (message in sw_last_error)       */
  SW_ESTATE = -4,       /* object used with the wrong handle / after free      */
  SW_EUNSUPPORTED = -5  /* valid request outside what this build supports      */
};

enum { SW_FLAG_TIMING = 1 }; /* sw_init flags: record CUDA events around kernels */

/* Create a handle on CUDA device `device`.  flags: SW_FLAG_* bits. */
int32_t sw_init(int32_t device, uint32_t flags, sw_handle_t* out);

/*
 * Pack and upload a database (host packer; the paper's
 * random-access binary format, L529-539).
 *   codes       host, residue codes, codes[offsets[d] .. offsets[d+1]) is
 *               sequence d; every code must be < alphabet_size.
 *   offsets     host, int64[n_seqs + 1], non-decreasing, offsets[0] may be > 0.
 *   n_seqs      >= 0; sequences of length 0 are allowed and score 0.
 *   alphabet_size  1..32; code alphabet_size is used internally as PAD.
 *   out         receives the DB; free with sw_free_db (or sw_free).
 * The inputs are copied; the call returns when the upload is complete.
 * Errors: SW_EINVAL (null pointer, bad offsets, code >= alphabet_size,
 * alphabet_size out of range), SW_ENOMEM, SW_ECUDA, SW_EUNSUPPORTED (a sequence
 * longer than 2^20 - 128 residues; UniProt's longest has 35,213, L762-764).
 */
int32_t sw_load_db(sw_handle_t h, const uint8_t* codes, const int64_t* offsets, int64_t n_seqs,
                   int32_t alphabet_size, void* cuda_stream, sw_db_t* out);

/*
 * sw_load_db with an output mapping (the scoring epilogue writes a
 * shard's scores straight into the full matrix, e.g. rank 0's buffer mapped into
 * this process over NVLink with CUDA IPC, so no gather collective follows).
 *   out_index   host, int64[n_seqs]: distinct output columns in [0, out_n).
 *   out_n       columns of the output rows (>= n_seqs).
 * sw_search on such a DB treats `scores` as int32[n_queries][out_n] (device or
 * peer-mapped memory only) and writes only this DB's columns (every one of
 * them, in every query row, including the zero rows of empty queries), leaving
 * the others untouched.  sw_align keeps the caller's local DB indices.
 * Errors: as sw_load_db; SW_EINVAL for a bad mapping.
 */
int32_t sw_load_db_mapped(sw_handle_t h, const uint8_t* codes, const int64_t* offsets, int64_t n_seqs,
                          int32_t alphabet_size, const int64_t* out_index, int64_t out_n, void* cuda_stream,
                          sw_db_t* out);

/*
 * Score every (query, database sequence) pair.
 *   q_codes, q_offsets   host, queries in the same layout as sw_load_db
 *                        (int64 q_offsets[n_queries + 1]); codes < alphabet.
 *   matrix      host, int8[alphabet_size * alphabet_size], row-major,
 *               matrix[a * alphabet_size + b] = S(query letter a, db letter b)
 *               (S_ij scores query element i vs element j).
 *   gap_open    Gs >= 0;  gap_extend  Ge >= 0;  Gs + Ge <= 32767.
 *   scores      host or device, int32[n_queries][n_seqs], row-major, in the
 *               caller's database order (the packer's length sort is undone).
 * Device `scores`: the call is stream-ordered on cuda_stream and never blocks
 * the host on the device (the int32 re-score kernel is always enqueued and reads
 * the flagged-pair count on the device); the caller synchronizes.  Host
 * `scores`: the call returns after the results are copied.
 * Streams: the handle's scratch is shared by its searches; a search waits (on
 * the device, cudaStreamWaitEvent) for the previous search of the same handle
 * when that one ran on another stream, so concurrent calls on different streams
 * are serialised on the device, never raced.  One host thread per handle.
 * Exactness: scores are exact int32; the int16 DPX path flags any pair whose
 * maximum reaches 32767 - max(matrix) and re-scores it in int32.
 * Errors: SW_EINVAL, SW_ESTATE (db from another handle), SW_ENOMEM, SW_ECUDA,
 * SW_EUNSUPPORTED (a query longer than 2^19 = 524,288 residues; the longest
 * UniProt protein, has 35,213).
 * n_queries == 0 or an empty DB is valid and writes nothing.
 */
int32_t sw_search(sw_handle_t h, const uint8_t* q_codes, const int64_t* q_offsets, int32_t n_queries,
                  sw_db_t db, const int8_t* matrix, int32_t gap_open, int32_t gap_extend, int32_t* scores,
                  void* cuda_stream);

/*
 * Best local alignment of selected (query, database sequence) pairs -- its
 * score, end cell, start cell and path (every
 * matrix element "keeps the cell that was used to produce the value", followed
 * back from the maximal cell).  Typical use: the top hits of an sw_search.
 *   q_codes, q_offsets, n_queries   host, queries as for sw_search.
 *   db          a DB loaded on this handle.
 *   pairs       host, int32[n_pairs][2] = (query index, DB sequence index in the
 *               caller's order).
 *   matrix, gap_open, gap_extend    as for sw_search.
 *   out5        host, int32[n_pairs][5] = {score, q_begin, q_end, d_begin, d_end}:
 *               0-based inclusive residue ranges of the alignment; all four -1
 *               when the score is 0 (no alignment).
 *   ops         host, uint32 run-length operations (len << 2 | op), op 0 = M
 *               (aligned pair), 1 = I (query residue vs gap), 2 = D (DB residue vs
 *               gap), start to end; pair k uses ops[ops_offsets[k] ..
 *               ops_offsets[k+1]) and n_ops[k] (host, int32[n_pairs]) receives
 *               the count.  A region of m_q + n_d entries always suffices.
 *   ops_offsets host, int64[n_pairs + 1], non-decreasing.
 * Tie-breaks (R-13): end cell = maximal H with the smallest DB position,
 * then the smallest query position; traceback prefers the diagonal, then E
 * (gap in the query), then F; a gap is opened rather than extended on a tie.
 * Synchronous: returns after the results are in the host buffers.
 * Scores are exact int32 (no int16 path).  Work: int32 wavefront kernel with a
 * 4-bit traceback code per cell kept in device memory (m*n/2 bytes per pair,
 * batched under the "align_workspace_mb" option), then one thread per pair
 * walks it.
 * Errors: SW_EINVAL (bad index, code, gaps, null pointer, a region too small
 * for the path), SW_ESTATE, SW_ENOMEM, SW_ECUDA, SW_EUNSUPPORTED (a DB sequence
 * longer than 2^20 - 64 or a query longer than 2^19).
 */
int32_t sw_align(sw_handle_t h, const uint8_t* q_codes, const int64_t* q_offsets, int32_t n_queries, sw_db_t db,
                 const int32_t* pairs, int32_t n_pairs, const int8_t* matrix, int32_t gap_open, int32_t gap_extend,
                 int32_t* out5, uint32_t* ops, const int64_t* ops_offsets, int32_t* n_ops, void* cuda_stream);

/*
 * CPU-type processing element of the hybrid SWDUAL (PAPER.md
 * sec. III: tasks are placed on "m CPUs and k GPUs" by the dual
 * approximation, sw_schedule_dual).  Host-only, no handle, no GPU: scores
 * n_queries x n_seqs pairs on n_threads host threads with a striped AVX2 int16
 * kernel (saturation-flagged pairs re-scored in int32) -- the work the paper's
 * CPU workers do (L529-539).  This is a scheduling target the caller chooses
 * for some tasks, never a fallback of sw_search.
 *   q_codes, q_offsets, n_queries   host, as for sw_search.
 *   db_codes, db_offsets, n_seqs    host, as for sw_load_db (not packed).
 *   alphabet_size, matrix, gap_open, gap_extend   as for sw_load_db / sw_search.
 *   n_threads   >= 1.
 *   scores      host, int32[n_queries][n_seqs].
 * Synchronous.  Errors: SW_EINVAL (as sw_search), SW_EUNSUPPORTED (no AVX2).
 */
int32_t sw_search_cpu(const uint8_t* q_codes, const int64_t* q_offsets, int32_t n_queries, const uint8_t* db_codes,
                      const int64_t* db_offsets, int64_t n_seqs, int32_t alphabet_size, const int8_t* matrix,
                      int32_t gap_open, int32_t gap_extend, int32_t n_threads, int32_t* scores);

/*
 * Merge of gathered score blocks into the full matrix (the
 * master "merge[s]" the workers' results).  After the
 * multi-GPU gather every rank's int32 blocks sit in one device buffer `src`;
 * block b holds blocks[b].n_rows x blocks[b].n_cols scores (row-major) at
 * src[src_off ..], its row i is query rows[row_off + i] and its column k is DB
 * sequence cols[col_off + k] of the caller's order.  sw_assemble writes
 * out[rows[..] * N + cols[..]] for every element, one kernel launch,
 * stream-ordered; elements of `out` covered by no block are left untouched.
 *   sw_assembly_create  host tables, copied to the device once (the layout is
 *                       fixed for a placement); rows in [0, n_queries), cols in
 *                       [0, N).  Free with sw_assembly_free (or sw_free).
 *   sw_assemble         src: device int32[src_len] (>= every block's end);
 *                       out: device int32[n_queries][N].
 * Errors: SW_EINVAL (bad table, index out of range, src too short, NULL),
 * SW_ENOMEM, SW_ECUDA.
 */
typedef struct sw_assembly_s* sw_assembly_t;
typedef struct {
  int64_t src_off, row_off, col_off, n_rows, n_cols;
} sw_block_t;
int32_t sw_assembly_create(sw_handle_t h, const sw_block_t* blocks, int32_t n_blocks, const int32_t* rows,
                           int64_t n_rows, const int64_t* cols, int64_t n_cols, int32_t n_queries, int64_t N,
                           sw_assembly_t* out);
int32_t sw_assemble(sw_assembly_t a, const int32_t* src, int64_t src_len, int32_t* out, void* cuda_stream);
int32_t sw_assembly_free(sw_assembly_t a);

int32_t sw_free_db(sw_db_t db);
int32_t sw_free(sw_handle_t h); /* frees the handle and any DBs still attached */

/* Message for the last failing call on h (or of the calling thread if h is NULL). */
const char* sw_last_error(sw_handle_t h);

/* --- introspection / tuning (not needed for plain use) ------------------- */

typedef struct {
  int64_t n_seqs, n_residues, n_pairs, n_long_pairs, max_len;
  int32_t alphabet_size, device;
} sw_db_info_t;
int32_t sw_db_info(sw_db_t db, sw_db_info_t* out);

typedef struct {
  double cells;            /* sum_q m_q * sum_d n_d of the last search (real residues)      */
  double cells_short;      /* of which scored by the short-pair (inter-task) kernels         */
  double cells_computed;   /* cell updates issued incl. row/column padding and wave fill     */
  double short_ms;         /* summed CUDA-event time of the short-pair kernel launches        */
  double long_ms;          /* CUDA-event time of the long-pair (intra-task) kernel, which    */
                           /* runs concurrently with them on the handle's side stream       */
  double search_ms;        /* device time of the whole search, first upload to last kernel   */
  int32_t n_launches;      /* kernels launched by the last search                           */
  int32_t n_score_launches;/* of which scoring (inter-task) kernels                         */
  int32_t n_overflow;      /* pairs re-scored in int32                                      */
  int32_t timing_valid;    /* 1 if the handle had SW_FLAG_TIMING / "timing" set              */
  int32_t last_G, last_R;  /* lane-group geometry of the last short-pair launch             */
} sw_stats_t;
/* Stats of the last sw_search; synchronizes the last search's stream. */
int32_t sw_last_stats(sw_handle_t h, sw_stats_t* out);

/*
 * Integer options (testing / tuning).  Keys:
 *   "overflow_threshold"  force the int16 re-score threshold (0 = automatic)
 *   "force_G", "force_R"  force the inter-task lane-group geometry of both short-pair
 *                         kernels (0 = auto; G in {4, 8, 16, 32}, R in {8, 12, .., 32})
 *   "query_pairs"         1 (default): queries are paired two per s16x2 register for
 *                         the short DB pairs (no PRMT); 0: one query per register
 *   "t_long"              >= 0: DB pairs longer than this are always scored in the
 *                         intra-task mode (whole CTAs on one pair); default -1:
 *                         automatic (pairs whose one-lane-group critical path
 *                         would outlast the search's average share, and every
 *                         pair > 3000 when such pairs hold most of the residues)
 *   "bank_copy"           1: shared-memory strip profiles as bank-spread copies
 *                         with 128-byte letter rows (default 1), 0: one copy
 *   "pack_queries"        1: a query-pair slot's shorter half carries further
 *                         queries laid end to end on strip boundaries (default 1)
 *   "bank_skew"           1: single-query profile copies one per lane group of
 *                         a shared-memory phase at searched bank skews
 *                         (conflict-free; default 1), 0: the linear layout
 *   "rescore_rows"        rows per lane of the int32 re-score: 0 (default) = 4 when every
 *                         query has fewer than 2^11 strips of 128 rows, else 8; 8 forces 8
 *   "const_gaps"          1 (default): searches with Gs = 10, Ge = 2 use kernel
 *                         instantiations with the penalties as immediates; 0: the
 *                         runtime-penalty kernels (same results)
 *   "timing"              1/0, same as SW_FLAG_TIMING
 *   "timing_accumulate"   1: short_ms/long_ms of sw_last_stats sum every search
 *                         since the last "timing_reset" (0: the last search only)
 *   "timing_reset"        clear the accumulated kernel events
 *   "align_workspace_mb"  device memory for sw_align's traceback codes per batch
 *                         (default 2048; a pair needing more runs alone)
 */
int32_t sw_set_option(sw_handle_t h, const char* key, int64_t value);

/* ASCII -> NCBI protein codes "ARNDCQEGHILKMFPSTWYVBZX*" (lower case folded, unknown -> X). */
int32_t sw_encode_ascii(const char* s, int64_t n, uint8_t* out);

/*
 * ASCII -> nucleotide codes (DNA over
 * {A, T, G, C}, RNA over {A, U, G, C}): A 0, C 1, G 2, T and U 3, anything else
 * (N, IUPAC ambiguity letters) 4; lower case folded.  Alphabet size 5: load the
 * DB with alphabet_size = 5 and score with a 5 x 5 match/mismatch matrix (the
 * paper's ma / mi, L127-133; the Python binding's nucleotide_matrix); the
 * linear gap g of Eq. (1) (L159-165) is gap_open = 0, gap_extend = -g.
 * s, out host; out may alias s.  Errors: SW_EINVAL (n < 0, NULL with n > 0).
 */
int32_t sw_encode_nucleotide(const char* s, int64_t n, uint8_t* out);

/*
 * Dual-approximation placement (sec. III): n_tasks tasks,
 * task j takes p_cpu[j] on a CPU-type PE and p_gpu[j] on a GPU-type PE
 * (host arrays, >= 0).  n_cpu >= 0 CPU PEs, n_gpu >= 0 GPU PEs, n_cpu+n_gpu >= 1.
 * Binary search on the guess lambda (L468-481); per guess: greedy knapsack by
 * decreasing p_cpu/p_gpu filling the GPUs up to area k*lambda (L370-387), the
 * rest on CPUs, list scheduling on each side (L388-396); "NO" when the CPU area
 * exceeds m*lambda.  out_pe[j] (host, int32[n_tasks]) = PE index, CPUs first
 * (0..n_cpu-1) then GPUs (n_cpu..n_cpu+n_gpu-1).  out_makespan / out_lambda may
 * be NULL.  Makespan <= 2 * lambda (Proposition 1).
 */
int32_t sw_schedule_dual(int64_t n_tasks, const double* p_cpu, const double* p_gpu, int32_t n_cpu,
                         int32_t n_gpu, int32_t* out_pe, double* out_makespan, double* out_lambda);

/*
 * The dynamic-programming variant of the same binary search (PAPER.md L482-502:
 * counting the tasks "with processing times larger than" a fraction of lambda and
 * solving the knapsack "via dynamic programming" brings the guarantee towards
 * 3/2 OPT; reading S-8).  Per guess: a task is big on a side when it
 * takes > lambda/2 there; the DP assigns sides minimising the CPU area with at
 * most n_cpu CPU-big and n_gpu GPU-big tasks and GPU area <= n_gpu * lambda (GPU
 * times rounded down to lambda / (4 n_tasks)); LPT on each side.  Makespan
 * <= (3/2 + 1/(4 n_gpu)) * lambda.  Same arguments and outputs as
 * sw_schedule_dual.  Time O(n^2 m k^2) per guess: SW_EUNSUPPORTED when the DP
 * table would exceed ~2.6e8 states (one byte each); SW_ENOMEM if the host
 * allocation fails (no C++ exception crosses the ABI).
 */
int32_t sw_schedule_dual_dp(int64_t n_tasks, const double* p_cpu, const double* p_gpu, int32_t n_cpu,
                            int32_t n_gpu, int32_t* out_pe, double* out_makespan, double* out_lambda);

/*
 * Host packer only (no device work): the packed form sw_load_db uploads.
 * Non-empty sequences sorted by length (longest first, ties by index), paired
 * neighbours (id1 = -1 for an odd leftover), each pair interleaved into 16-bit
 * words code(id0) | code(id1) << 8 over `len` columns (multiple of 4, PAD =
 * alphabet_size), pair p at stream[off .. off+len).  Pairs [0, n_long) are
 * longer than t_long.  Two-phase: pass pairs == NULL and stream == NULL to get
 * *n_pairs and *stream_words, then call again with buffers of those sizes.
 * Errors: SW_EINVAL as for sw_load_db.
 */
typedef struct {
  int64_t off;
  int32_t len, id0, id1, pad_;
} sw_pair_t;
int32_t sw_pack_db_host(const uint8_t* codes, const int64_t* offsets, int64_t n_seqs, int32_t alphabet_size,
                        int64_t t_long, sw_pair_t* pairs, int64_t* n_pairs, uint16_t* stream,
                        int64_t* stream_words, int64_t* n_long);

/*
 * Host-only gather of selected sequences (the multi-GPU layer's shard cut, SURVEY
 * 8(a) a3): sequences ids[0..n_ids) of (codes, offsets[n_seqs + 1]) are copied, in
 * that order, to out_codes with out_offsets[n_ids + 1] (starting at 0).  Two-phase:
 * with out_codes == NULL only *n_out (residues) and, if given, out_offsets are
 * written.  Host threads, no device work.  Errors: SW_EINVAL (index out of range,
 * bad offsets, NULL), SW_ENOMEM.
 */
int32_t sw_subset_host(const uint8_t* codes, const int64_t* offsets, int64_t n_seqs, const int64_t* ids,
                       int64_t n_ids, uint8_t* out_codes, int64_t* out_offsets, int64_t* n_out);

#ifdef __cplusplus
}
#endif
#endif /* SWDUAL_H */
