// Dual-approximation placement of tasks on CPU-type and GPU-type processing
// elements -- the SWDUAL scheduler (sec. III).
//
//   g-dual approximation, g = 2 (L315-326): for a guess lambda either return a
//   schedule of makespan <= 2*lambda or answer "NO" (no schedule <= lambda).
//   Per guess (L340-396):
//     * a task longer than lambda on one side must go to the other side; longer
//       than lambda on both -> NO ("the execution time of each task is at most
//       lambda", L344);
//     * greedy min-knapsack (Eqs. (5)-(7), L353-387): tasks by decreasing
//       p_cpu/p_gpu (reading S-2) fill the GPUs until their area
//       reaches k*lambda (the last one overshoots, L378-379); the rest go to the
//       CPUs; CPU area > m*lambda -> NO (constraint (C1), L349-350);
//     * list scheduling on each side (L388-396): longest task first onto the
//       least-loaded PE of its type (reading S-4).
//   Binary search on lambda between Bmin and Bmax (L468-481, reading S-5).
// With m = 0 CPUs (the B200 box, reading S-6) every task is a GPU task and the
// method reduces to binary search + LPT list scheduling.
#include <new>
#include <algorithm>
#include <cmath>
#include <limits>
#include <cstdint>
#include <numeric>
#include <vector>

#include "../../include/swdual.h"

namespace {

struct Sched {
  std::vector<int32_t> pe;
  double makespan = 0;
};

// LPT list scheduling of `tasks` (indices) with times `p` onto `npe` PEs whose
// global indices start at `base`; returns the max load.
double list_schedule(const std::vector<int64_t>& tasks, const double* p, int npe, int base, std::vector<int32_t>& pe) {
  if (tasks.empty()) return 0.0;
  std::vector<int64_t> order(tasks);
  std::stable_sort(order.begin(), order.end(), [&](int64_t a, int64_t b) { return p[a] > p[b]; });
  std::vector<double> load(size_t(npe), 0.0);
  for (int64_t j : order) {
    int best = 0;
    for (int q = 1; q < npe; ++q)
      if (load[size_t(q)] < load[size_t(best)]) best = q;
    load[size_t(best)] += p[j];
    pe[size_t(j)] = base + best;
  }
  return *std::max_element(load.begin(), load.end());
}

// One dual-approximation step for guess lam.  Returns false for "NO".
bool dual_step(int64_t n, const double* pc, const double* pg, int m, int k, double lam, Sched& out) {
  out.pe.assign(size_t(n), -1);
  std::vector<int64_t> cpu, gpu, free_;
  double WG = 0, WC = 0;
  for (int64_t j = 0; j < n; ++j) {
    const bool cpu_ok = m > 0 && pc[j] <= lam;
    const bool gpu_ok = k > 0 && pg[j] <= lam;
    if (!cpu_ok && !gpu_ok) return false;
    if (!cpu_ok) { gpu.push_back(j); WG += pg[j]; }
    else if (!gpu_ok) { cpu.push_back(j); WC += pc[j]; }
    else free_.push_back(j);
  }
  if (k > 0 && WG > k * lam) return false;  // forced GPU tasks alone exceed the GPU area
  // greedy knapsack: decreasing p_cpu / p_gpu (GPU-friendliest first), ties by index
  std::stable_sort(free_.begin(), free_.end(), [&](int64_t a, int64_t b) {
    // compare pc[a]/pg[a] > pc[b]/pg[b] without dividing by zero
    return pc[a] * pg[b] > pc[b] * pg[a];
  });
  size_t i = 0;
  if (k > 0)
    for (; i < free_.size() && WG < k * lam; ++i) { gpu.push_back(free_[i]); WG += pg[free_[i]]; }
  for (; i < free_.size(); ++i) { cpu.push_back(free_[i]); WC += pc[free_[i]]; }
  if (WC > m * lam + 1e-12 * std::max(1.0, WC)) return false;
  const double mc = list_schedule(cpu, pc, m, 0, out.pe);
  const double mg = list_schedule(gpu, pg, k, m, out.pe);
  out.makespan = std::max(mc, mg);
  return true;
}

// One step of the DP-knapsack variant for guess lam ("constraints
// on the number of tasks with processing times larger than" a fraction of lambda,
// solved "via dynamic programming", after [13]; reading S-8).  A task is
// big on a side when it takes more than lam/2 there; a schedule of makespan <= lam
// holds at most m big tasks on the CPUs and k on the GPUs.  The DP chooses the side
// of every task minimising the CPU area under those counts and the GPU area <= k*lam
// (GPU times rounded down to lam/(4n): a feasible lam is never rejected).  Then LPT
// list scheduling on each side: the bigs land alone first, any later task starts
// below the average load, so CPUs end by 3/2 lam and GPUs by (3/2 + 1/(4k)) lam.
bool dual_step_dp(int64_t n, const double* pc, const double* pg, int m, int k, double lam, Sched& out) {
  constexpr int GRID = 4;
  out.pe.assign(size_t(n), -1);
  const double half = 0.5 * lam;
  const double delta = lam / (double(GRID) * double(n));
  const int64_t cap = k > 0 ? int64_t(k) * GRID * n : 0;
  const int64_t M1 = m + 1, K1 = k + 1, C1 = cap + 1;
  const int64_t S = M1 * K1 * C1;
  const double INF = std::numeric_limits<double>::infinity();
  std::vector<double> cur(static_cast<size_t>(S), INF), nxt(static_cast<size_t>(S), INF);
  std::vector<uint8_t> choice(size_t(n) * size_t(S), 0);  // 1 = task on a GPU
  cur[0] = 0.0;
  auto idx = [&](int64_t mu, int64_t ka, int64_t g) { return (mu * K1 + ka) * C1 + g; };
  for (int64_t j = 0; j < n; ++j) {
    std::fill(nxt.begin(), nxt.end(), INF);
    const bool cpu_ok = m > 0 && pc[j] <= lam, gpu_ok = k > 0 && pg[j] <= lam;
    if (!cpu_ok && !gpu_ok) return false;
    const int bc = pc[j] > half ? 1 : 0, bg = pg[j] > half ? 1 : 0;
    const int64_t r = gpu_ok ? int64_t(std::floor(pg[j] / delta)) : 0;
    uint8_t* ch = choice.data() + size_t(j) * size_t(S);
    for (int64_t mu = 0; mu < M1; ++mu)
      for (int64_t ka = 0; ka < K1; ++ka)
        for (int64_t g = 0; g < C1; ++g) {
          const double w = cur[size_t(idx(mu, ka, g))];
          if (w == INF) continue;
          if (cpu_ok && mu + bc < M1) {
            const int64_t t = idx(mu + bc, ka, g);
            if (w + pc[j] < nxt[size_t(t)]) { nxt[size_t(t)] = w + pc[j]; ch[t] = 0; }
          }
          if (gpu_ok && ka + bg < K1 && g + r < C1) {
            const int64_t t = idx(mu, ka + bg, g + r);
            if (w < nxt[size_t(t)]) { nxt[size_t(t)] = w; ch[t] = 1; }
          }
        }
    cur.swap(nxt);
  }
  int64_t bst = -1;
  for (int64_t t = 0; t < S; ++t)
    if (cur[size_t(t)] != INF && (bst < 0 || cur[size_t(t)] < cur[size_t(bst)])) bst = t;
  if (bst < 0 || cur[size_t(bst)] > m * lam + 1e-12 * std::max(1.0, cur[size_t(bst)])) return false;
  // walk the choices back from the best final state
  std::vector<int64_t> cpu, gpu;
  int64_t mu = bst / (K1 * C1), ka = (bst / C1) % K1, g = bst % C1;
  for (int64_t j = n - 1; j >= 0; --j) {
    const int64_t t = idx(mu, ka, g);
    if (choice[size_t(j) * size_t(S) + size_t(t)]) {
      gpu.push_back(j);
      ka -= pg[j] > half ? 1 : 0;
      g -= int64_t(std::floor(pg[j] / delta));
    } else {
      cpu.push_back(j);
      mu -= pc[j] > half ? 1 : 0;
    }
  }
  const double mc = list_schedule(cpu, pc, m, 0, out.pe);
  const double mg = list_schedule(gpu, pg, k, m, out.pe);
  out.makespan = std::max(mc, mg);
  return true;
}

using step_fn = bool (*)(int64_t, const double*, const double*, int, int, double, Sched&);

int32_t binary_search(step_fn step, int64_t n_tasks, const double* p_cpu, const double* p_gpu, int32_t n_cpu,
                      int32_t n_gpu, int32_t* out_pe, double* out_makespan, double* out_lambda);

}  // namespace

namespace {
int32_t binary_search(step_fn step, int64_t n_tasks, const double* p_cpu, const double* p_gpu, int32_t n_cpu,
                      int32_t n_gpu, int32_t* out_pe, double* out_makespan, double* out_lambda) {
  if (n_tasks < 0 || n_cpu < 0 || n_gpu < 0 || n_cpu + n_gpu < 1) return SW_EINVAL;
  if (n_tasks > 0 && (!p_cpu || !p_gpu || !out_pe)) return SW_EINVAL;
  for (int64_t j = 0; j < n_tasks; ++j)
    if (!(p_cpu[j] >= 0) || !(p_gpu[j] >= 0) || !std::isfinite(p_cpu[j]) || !std::isfinite(p_gpu[j]))
      return SW_EINVAL;
  if (n_tasks == 0) {
    if (out_makespan) *out_makespan = 0;
    if (out_lambda) *out_lambda = 0;
    return SW_OK;
  }
  const int m = n_cpu, k = n_gpu;
  // Bmin: every task takes at least min(p, pbar); total area spread on m + k PEs
  double mx = 0, area = 0;
  for (int64_t j = 0; j < n_tasks; ++j) {
    double lo;
    if (m == 0) lo = p_gpu[j];
    else if (k == 0) lo = p_cpu[j];
    else lo = std::min(p_cpu[j], p_gpu[j]);
    mx = std::max(mx, lo);
    area += lo;
  }
  double lo = std::max(mx, area / double(m + k));
  // Bmax: a feasible schedule -- all tasks on the PE type with more PEs... take
  // the list schedule on the faster side per task, then double until accepted.
  Sched best, cur;
  double hi = std::max(lo, 1e-300);
  while (!step(n_tasks, p_cpu, p_gpu, m, k, hi, cur)) hi *= 2;
  best = cur;
  double lam_acc = hi;
  for (int it = 0; it < 64 && hi - lo > 1e-4 * hi; ++it) {
    const double lam = 0.5 * (lo + hi);
    if (step(n_tasks, p_cpu, p_gpu, m, k, lam, cur)) {
      hi = lam;
      lam_acc = lam;
      if (cur.makespan <= best.makespan) best = cur;
    } else {
      lo = lam;
    }
  }
  for (int64_t j = 0; j < n_tasks; ++j) out_pe[j] = best.pe[size_t(j)];
  if (out_makespan) *out_makespan = best.makespan;
  if (out_lambda) *out_lambda = lam_acc;
  return SW_OK;
}
}  // namespace

// No C++ exception may cross the C ABI: a failed host allocation becomes SW_ENOMEM.
static int32_t guarded_search(step_fn step, int64_t n_tasks, const double* p_cpu, const double* p_gpu,
                              int32_t n_cpu, int32_t n_gpu, int32_t* out_pe, double* out_makespan,
                              double* out_lambda) {
  try {
    return binary_search(step, n_tasks, p_cpu, p_gpu, n_cpu, n_gpu, out_pe, out_makespan, out_lambda);
  } catch (const std::bad_alloc&) {
    return SW_ENOMEM;
  } catch (...) {
    return SW_EINVAL;
  }
}

extern "C" int32_t sw_schedule_dual(int64_t n_tasks, const double* p_cpu, const double* p_gpu, int32_t n_cpu,
                                    int32_t n_gpu, int32_t* out_pe, double* out_makespan, double* out_lambda) {
  return guarded_search(dual_step, n_tasks, p_cpu, p_gpu, n_cpu, n_gpu, out_pe, out_makespan, out_lambda);
}

extern "C" int32_t sw_schedule_dual_dp(int64_t n_tasks, const double* p_cpu, const double* p_gpu, int32_t n_cpu,
                                       int32_t n_gpu, int32_t* out_pe, double* out_makespan, double* out_lambda) {
  // the DP table holds (m+1)(k+1)(4kn+1) states per task
  const double states = double(n_cpu + 1) * double(n_gpu + 1) * (4.0 * double(n_gpu) * double(n_tasks) + 1.0);
  // (one byte of choice table per state and task, rebuilt per bisection step: <= 256 MB)
  if (n_tasks > 0 && states * double(n_tasks) > 2.56e8) return SW_EUNSUPPORTED;
  return guarded_search(dual_step_dp, n_tasks, p_cpu, p_gpu, n_cpu, n_gpu, out_pe, out_makespan, out_lambda);
}
