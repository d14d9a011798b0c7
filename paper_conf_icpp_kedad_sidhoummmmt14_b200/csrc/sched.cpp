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
#include <algorithm>
#include <cmath>
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

}  // namespace

extern "C" int32_t sw_schedule_dual(int64_t n_tasks, const double* p_cpu, const double* p_gpu, int32_t n_cpu,
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
  while (!dual_step(n_tasks, p_cpu, p_gpu, m, k, hi, cur)) hi *= 2;
  best = cur;
  double lam_acc = hi;
  for (int it = 0; it < 64 && hi - lo > 1e-4 * hi; ++it) {
    const double lam = 0.5 * (lo + hi);
    if (dual_step(n_tasks, p_cpu, p_gpu, m, k, lam, cur)) {
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
