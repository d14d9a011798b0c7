// Host packer: validate, length-sort, pair, interleave.
//
// The paper's binary database format gives random access to any sequence and
// known sizes up front; here the packed form is what the
// GPU kernels stream:
//   * non-empty sequences sorted by length, longest first, ties by caller index;
//   * neighbours paired: pair p = (sorted[2p], sorted[2p+1]); the s16x2 lanes
//     score both halves of a pair at once, so pairing equal lengths wastes
//     almost nothing;
//   * each pair interleaved column by column into 16-bit words
//     (low byte = id0's residue, high byte = id1's), padded to a multiple of 4
//     columns with PAD = alphabet_size, 4 columns = one 8-byte load;
//   * pairs [0, n_long) are longer than t_long (launched separately).
#include <cstring>
#include <algorithm>
#include <atomic>
#include <stdexcept>
#include <string>
#include <thread>
#include <vector>

#include "../../include/swdual.h"
#include "sw_internal.h"

namespace swdual {

static unsigned n_threads() { return std::max(1u, std::min(16u, std::thread::hardware_concurrency())); }
unsigned n_threads_host() { return n_threads(); }

void pack_db(const uint8_t* codes, const int64_t* offsets, int64_t n_seqs, int alpha, int64_t t_long, Packed& P,
             bool nib) {
  if (n_seqs < 0) throw std::invalid_argument("n_seqs < 0");
  if (alpha < 1 || alpha > 32) throw std::invalid_argument("alphabet_size must be in 1..32");
  if (n_seqs > 0 && !offsets) throw std::invalid_argument("offsets is NULL");
  if (n_seqs >= (int64_t(1) << 31) - 1) throw std::invalid_argument("more than 2^31-2 sequences");
  P = Packed{};
  P.seq_len.resize(size_t(n_seqs));
  int64_t total = 0;
  for (int64_t i = 0; i < n_seqs; ++i) {
    const int64_t L = offsets[i + 1] - offsets[i];
    if (L < 0) throw std::invalid_argument("offsets not non-decreasing");
    if (L > (int64_t(1) << 30)) throw std::invalid_argument("sequence longer than 2^30");
    P.seq_len[size_t(i)] = L;
    total += L;
  }
  if (total > 0 && !codes) throw std::invalid_argument("codes is NULL");
  P.n_res = total;
  if (total > 0) {  // every code < alpha (parallel scan)
    const uint8_t* base = codes + offsets[0];
    const unsigned nt = n_threads();
    std::atomic<bool> bad{false};
    std::vector<std::thread> th;
    for (unsigned t = 0; t < nt; ++t)
      th.emplace_back([&, t] {
        const int64_t a = total * t / nt, b = total * (t + 1) / nt;
        for (int64_t i = a; i < b; ++i)
          if (base[i] >= alpha) { bad = true; return; }
      });
    for (auto& x : th) x.join();
    if (bad) throw std::invalid_argument("residue code >= alphabet_size");
  }
  std::vector<int32_t> order;
  order.reserve(size_t(n_seqs));
  for (int64_t i = 0; i < n_seqs; ++i)
    if (P.seq_len[size_t(i)] > 0) order.push_back(int32_t(i));
  std::stable_sort(order.begin(), order.end(),
                   [&](int32_t a, int32_t b) { return P.seq_len[size_t(a)] > P.seq_len[size_t(b)]; });
  P.sorted_lens.resize(order.size());
  for (size_t i = 0; i < order.size(); ++i) P.sorted_lens[i] = P.seq_len[size_t(order[i])];
  P.max_len = order.empty() ? 0 : P.sorted_lens[0];
  const size_t np = (order.size() + 1) / 2;
  P.pairs.resize(np);
  int64_t off = 0;
  for (size_t p = 0; p < np; ++p) {
    PairRec& r = P.pairs[p];
    r.id0 = order[2 * p];
    r.id1 = (2 * p + 1 < order.size()) ? order[2 * p + 1] : -1;
    const int64_t L = P.seq_len[size_t(r.id0)];  // the longer of the two (sorted)
    r.len = int32_t((L + 3) / 4 * 4);
    r.off = off;
    r.pad_ = 0;
    off += r.len;
    if (L > t_long) P.n_long = int(p + 1);
  }
  if (nib && alpha > 15) throw std::invalid_argument("4-bit codes need alphabet_size <= 15");
  P.nib = nib ? 1 : 0;
  if (nib) {  // one byte per pair column: two 4-bit codes (PAD = alpha <= 15)
    P.stream.assign(size_t(std::max<int64_t>((off + 1) / 2, 4)), 0);
    uint8_t* bytes = reinterpret_cast<uint8_t*>(P.stream.data());
    std::fill(bytes, bytes + 2 * P.stream.size(), uint8_t(alpha | (alpha << 4)));
    const unsigned nt = n_threads();
    std::vector<std::thread> th;
    for (unsigned t = 0; t < nt; ++t)
      th.emplace_back([&, t] {
        for (size_t p = t; p < np; p += nt) {
          const PairRec& r = P.pairs[p];
          const uint8_t* s0 = codes + offsets[r.id0];
          const int64_t l0 = P.seq_len[size_t(r.id0)];
          const uint8_t* s1 = r.id1 >= 0 ? codes + offsets[r.id1] : nullptr;
          const int64_t l1 = r.id1 >= 0 ? P.seq_len[size_t(r.id1)] : 0;
          uint8_t* w = bytes + r.off;
          for (int64_t c = 0; c < r.len; ++c) {
            const uint8_t a = c < l0 ? s0[c] : uint8_t(alpha);
            const uint8_t b = c < l1 ? s1[c] : uint8_t(alpha);
            w[c] = uint8_t(a | (b << 4));
          }
        }
      });
    for (auto& x : th) x.join();
    return;
  }
  P.stream.assign(size_t(std::max<int64_t>(off, 4)), uint16_t(alpha | (alpha << 8)));
  const uint16_t pad = uint16_t(alpha);
  const unsigned nt = n_threads();
  std::vector<std::thread> th;
  for (unsigned t = 0; t < nt; ++t)
    th.emplace_back([&, t] {
      for (size_t p = t; p < np; p += nt) {
        const PairRec& r = P.pairs[p];
        const uint8_t* s0 = codes + offsets[r.id0];
        const int64_t l0 = P.seq_len[size_t(r.id0)];
        const uint8_t* s1 = r.id1 >= 0 ? codes + offsets[r.id1] : nullptr;
        const int64_t l1 = r.id1 >= 0 ? P.seq_len[size_t(r.id1)] : 0;
        uint16_t* w = P.stream.data() + r.off;
        for (int64_t c = 0; c < r.len; ++c) {
          const uint16_t a = c < l0 ? s0[c] : pad;
          const uint16_t b = c < l1 ? s1[c] : pad;
          w[c] = uint16_t(a | (b << 8));
        }
      }
    });
  for (auto& x : th) x.join();
}

}  // namespace swdual

// Host-only access to the packer (tests, tooling): two-phase, call with
// pairs == NULL / stream == NULL to get the sizes first.
extern "C" int32_t sw_pack_db_host(const uint8_t* codes, const int64_t* offsets, int64_t n_seqs, int32_t alphabet_size,
                                   int64_t t_long, sw_pair_t* pairs, int64_t* n_pairs, uint16_t* stream,
                                   int64_t* stream_words, int64_t* n_long) {
  static_assert(sizeof(sw_pair_t) == sizeof(swdual::PairRec), "sw_pair_t layout");
  try {
    swdual::Packed P;
    swdual::pack_db(codes, offsets, n_seqs, alphabet_size, t_long, P);
    if (n_pairs) *n_pairs = int64_t(P.pairs.size());
    if (stream_words) *stream_words = int64_t(P.stream.size());
    if (n_long) *n_long = P.n_long;
    if (pairs) std::copy(P.pairs.begin(), P.pairs.end(), reinterpret_cast<swdual::PairRec*>(pairs));
    if (stream) std::copy(P.stream.begin(), P.stream.end(), stream);
    return SW_OK;
  } catch (const std::invalid_argument&) {
    return SW_EINVAL;
  } catch (...) {
    return SW_ENOMEM;
  }
}

// Host-only gather of selected sequences (the shard cut of the multi-GPU layer):
// out_codes / out_offsets receive sequences ids[0..n_ids) in that order.  Two-phase:
// out_codes == NULL returns the residue count in *n_out (offsets are filled when
// out_offsets != NULL).  Copies run on the host's threads (C5 shards: billions of
// residues, where an index-array gather would need 8 bytes per residue).
extern "C" int32_t sw_subset_host(const uint8_t* codes, const int64_t* offsets, int64_t n_seqs, const int64_t* ids,
                                  int64_t n_ids, uint8_t* out_codes, int64_t* out_offsets, int64_t* n_out) {
  try {
    if (n_ids < 0 || n_seqs < 0 || (n_ids > 0 && !ids) || (n_seqs > 0 && !offsets)) return SW_EINVAL;
    std::vector<int64_t> off(size_t(n_ids) + 1, 0);
    for (int64_t k = 0; k < n_ids; ++k) {
      const int64_t d = ids[k];
      if (d < 0 || d >= n_seqs) return SW_EINVAL;
      const int64_t L = offsets[d + 1] - offsets[d];
      if (L < 0) return SW_EINVAL;
      off[size_t(k) + 1] = off[size_t(k)] + L;
    }
    if (n_out) *n_out = off.back();
    if (out_offsets) std::copy(off.begin(), off.end(), out_offsets);
    if (!out_codes) return SW_OK;
    if (off.back() > 0 && !codes) return SW_EINVAL;
    const unsigned nt = swdual::n_threads_host();
    std::vector<std::thread> th;
    for (unsigned t = 0; t < nt; ++t)
      th.emplace_back([&, t] {
        const int64_t a = n_ids * t / nt, b = n_ids * (t + 1) / nt;
        for (int64_t k = a; k < b; ++k)
          std::memcpy(out_codes + off[size_t(k)], codes + offsets[ids[k]], size_t(off[size_t(k) + 1] - off[size_t(k)]));
      });
    for (auto& x : th) x.join();
    return SW_OK;
  } catch (...) {
    return SW_ENOMEM;
  }
}
