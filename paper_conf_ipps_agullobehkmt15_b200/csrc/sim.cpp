// Host-side platform model of PAPER.md §III-IV: the makespan lower
// bound LP over several resource types (area bound L349-359, mixed bound L388-404) and
// a discrete-event replay of the Algorithm 1 task DAG on a platform of resource classes
// (CPU cores, GPUs, ...) under the paper's schedulers -- dmda (minimum completion time,
// L645-651), dmdas (the same in bottom-level priority order, L652-660) -- and its static
// rules (GEMM/SYRK forced on one class, L1000-1007; TRSMs at least d tiles below the
// diagonal forced on another, L1019-1025).  The paper runs these experiments in
// StarPU-SimGrid (L582-631); this is the same model without data transfers (the B200
// path moves operands through L2/NVLink, overlapped; reading R18).
#include <algorithm>
#include <cmath>
#include <cstdint>
#include <queue>
#include <vector>

#include "../../include/chol.h"
#include "dag.h"
#include "taskid.h"

namespace chol {
namespace {

// Dense two-phase simplex (Bland's rule) for  min c.x  s.t.  A x = b (b >= 0), x >= 0.
// Sizes here are tiny (<= 9 rows, <= 40 columns).  Returns 0 on success, 1 infeasible,
// 2 unbounded.
int simplex(std::vector<std::vector<double>> A, std::vector<double> b, const std::vector<double>& c,
            std::vector<double>& x) {
  const int m = (int)A.size(), n = (int)c.size();
  const double eps = 1e-9;
  // tableau: n structural + m artificial columns, rhs last
  const int W = n + m + 1;
  std::vector<std::vector<double>> T(m + 1, std::vector<double>(W, 0.0));
  std::vector<int> basis(m);
  for (int r = 0; r < m; ++r) {
    for (int j = 0; j < n; ++j) T[r][j] = A[r][j];
    T[r][n + r] = 1.0;
    T[r][W - 1] = b[r];
    basis[r] = n + r;
  }
  auto pivot = [&](int pr, int pc) {
    const double pv = T[pr][pc];
    for (double& v : T[pr]) v /= pv;
    for (int r = 0; r <= m; ++r)
      if (r != pr && T[r][pc] != 0.0) {
        const double f = T[r][pc];
        for (int j = 0; j < W; ++j) T[r][j] -= f * T[pr][j];
      }
    basis[pr] = pc;
  };
  auto run = [&](int ncols) -> int {  // objective row m holds reduced costs (minimise)
    for (int it = 0; it < 10000; ++it) {
      int pc = -1;
      for (int j = 0; j < ncols; ++j)
        if (T[m][j] < -eps) {
          pc = j;
          break;
        }
      if (pc < 0) return 0;
      int pr = -1;
      double best = 0.0;
      for (int r = 0; r < m; ++r)
        if (T[r][pc] > eps) {
          const double ratio = T[r][W - 1] / T[r][pc];
          if (pr < 0 || ratio < best - eps || (std::fabs(ratio - best) <= eps && basis[r] < basis[pr])) {
            pr = r;
            best = ratio;
          }
        }
      if (pr < 0) return 2;
      pivot(pr, pc);
    }
    return 2;
  };
  // phase 1: minimise the sum of the artificials
  for (int j = 0; j < W; ++j) T[m][j] = 0.0;
  for (int r = 0; r < m; ++r)
    for (int j = 0; j < W; ++j)
      if (j < n || j == W - 1) T[m][j] -= T[r][j];
  if (run(n + m) != 0) return 1;
  if (-T[m][W - 1] > 1e-7 * (1.0 + std::fabs(T[m][W - 1]))) return 1;
  // drive remaining artificials out of the basis where possible
  for (int r = 0; r < m; ++r)
    if (basis[r] >= n)
      for (int j = 0; j < n; ++j)
        if (std::fabs(T[r][j]) > eps) {
          pivot(r, j);
          break;
        }
  // phase 2 over the structural columns
  for (int j = 0; j < W; ++j) T[m][j] = 0.0;
  for (int j = 0; j < n; ++j) T[m][j] = c[j];
  for (int r = 0; r < m; ++r)
    if (basis[r] < n && c[basis[r]] != 0.0) {
      const double f = c[basis[r]];
      for (int j = 0; j < W; ++j) T[m][j] -= f * T[r][j];
    }
  const int st = run(n);
  if (st) return st;
  x.assign(n, 0.0);
  for (int r = 0; r < m; ++r)
    if (basis[r] < n) x[basis[r]] = T[r][W - 1];
  return 0;
}

bool runs_on(const chol_sim_opts_t& o, int cls, int type, int i, int k) {
  const double t = o.time[cls][type];
  if (!(t >= 0.0) || std::isinf(t)) return false;
  if (o.gemm_syrk_class >= 0 && (type == T_SYRK || type == T_GEMM) && cls != o.gemm_syrk_class) return false;
  if (o.trsm_far_class >= 0 && type == T_TRSM && i - k >= o.trsm_far_distance && cls != o.trsm_far_class)
    return false;
  return true;
}

}  // namespace
}  // namespace chol

using namespace chol;

extern "C" int chol_lp_bound(int64_t N, int nclasses, const int* workers, const double* time, int mixed,
                             double* l_out, double* n_rt) {
  if (N <= 0) return -1;
  if (nclasses < 1 || nclasses > CHOL_SIM_MAX_CLASSES || !workers || !time || !l_out) return -6;
  const int R = nclasses;
  const double cnt[4] = {(double)N, (double)n_trsm(N), (double)n_trsm(N), (double)n_gemm(N)};
  // variables: x_rt for runnable (r, t), then l, then slacks (R, + 1 if mixed)
  std::vector<int> var_r, var_t;
  for (int r = 0; r < R; ++r) {
    if (workers[r] < 0) return -6;
    for (int t = 0; t < 4; ++t) {
      const double v = time[r * 4 + t];
      if (v >= 0.0 && !std::isinf(v) && workers[r] > 0) {
        var_r.push_back(r);
        var_t.push_back(t);
      }
    }
  }
  const int nx = (int)var_r.size(), il = nx, is0 = nx + 1;
  const int nv = nx + 1 + R + (mixed ? 1 : 0);
  std::vector<std::vector<double>> A;
  std::vector<double> b;
  for (int t = 0; t < 4; ++t) {  // sum_r n_rt = N_t  (L352-354)
    std::vector<double> row(nv, 0.0);
    bool any = false;
    for (int v = 0; v < nx; ++v)
      if (var_t[v] == t) row[v] = 1.0, any = true;
    if (!any && cnt[t] > 0) return -6;  // a task type no class can run
    A.push_back(row);
    b.push_back(cnt[t]);
  }
  for (int r = 0; r < R; ++r) {  // sum_t n_rt T_rt - M_r l + s_r = 0  (L355-357)
    std::vector<double> row(nv, 0.0);
    for (int v = 0; v < nx; ++v)
      if (var_r[v] == r) row[v] = time[r * 4 + var_t[v]];
    row[il] = -(double)workers[r];
    row[is0 + r] = 1.0;
    A.push_back(row);
    b.push_back(0.0);
  }
  if (mixed) {  // sum_r n_rP T_rP + (N-1)(T*_T + T*_S) <= l   (L390-396), as  l - sum - s = C
    double tT = INFINITY, tS = INFINITY;
    for (int v = 0; v < nx; ++v) {
      const double tv = time[var_r[v] * 4 + var_t[v]];
      if (var_t[v] == T_TRSM) tT = std::min(tT, tv);
      if (var_t[v] == T_SYRK) tS = std::min(tS, tv);
    }
    if (N == 1) tT = tS = 0.0;
    std::vector<double> row(nv, 0.0);
    for (int v = 0; v < nx; ++v)
      if (var_t[v] == T_POTRF) row[v] = -time[var_r[v] * 4 + T_POTRF];
    row[il] = 1.0;
    row[nv - 1] = -1.0;
    A.push_back(row);
    b.push_back((double)(N - 1) * (tT + tS));
  }
  std::vector<double> c(nv, 0.0), x;
  c[il] = 1.0;
  const int st = simplex(A, b, c, x);
  if (st) return -6;
  *l_out = x[il];
  if (n_rt) {
    for (int i = 0; i < R * 4; ++i) n_rt[i] = 0.0;
    for (int v = 0; v < nx; ++v) n_rt[var_r[v] * 4 + var_t[v]] = x[v];
  }
  return 0;
}

extern "C" int chol_simulate(int64_t N, const chol_sim_opts_t* o, double* makespan, chol_task_rec_t* recs,
                             int64_t cap) {
  if (N <= 0) return -1;
  if (!o || !makespan) return -4;
  if (o->nclasses < 1 || o->nclasses > CHOL_SIM_MAX_CLASSES || o->policy < 0 || o->policy > 2) return -6;
  if (o->policy == CHOL_SIM_FIXED && (!o->fixed_worker || !o->fixed_rank)) return -4;
  const int R = o->nclasses;
  // workers, their classes
  std::vector<int> wcls;
  for (int r = 0; r < R; ++r) {
    if (o->workers[r] < 0) return -6;
    for (int w = 0; w < o->workers[r]; ++w) wcls.push_back(r);
  }
  const int W = (int)wcls.size();
  if (W == 0) return -6;
  std::vector<std::pair<int64_t, int64_t>> E;
  std::vector<int> type_of;
  build_task_dag(N, E, type_of);
  const int64_t nt = n_tasks(N);
  std::vector<int> ti(nt), tj(nt), tk(nt);  // chol_trace convention
  for (int64_t k = 0; k < N; ++k) {
    ti[id_potrf(N, k)] = (int)k, tj[id_potrf(N, k)] = (int)k, tk[id_potrf(N, k)] = (int)k;
    for (int64_t i = k + 1; i < N; ++i) {
      const int64_t t = id_trsm(N, i, k);
      ti[t] = (int)i, tj[t] = (int)k, tk[t] = (int)k;
    }
    for (int64_t j = k + 1; j < N; ++j) {
      int64_t t = id_syrk(N, j, k);
      ti[t] = (int)j, tj[t] = (int)j, tk[t] = (int)k;
      for (int64_t i = j + 1; i < N; ++i) {
        t = id_gemm(N, i, j, k);
        ti[t] = (int)i, tj[t] = (int)j, tk[t] = (int)k;
      }
    }
  }
  // every task must have a class that may run it
  for (int64_t t = 0; t < nt; ++t) {
    bool ok = false;
    for (int r = 0; r < R && !ok; ++r) ok = o->workers[r] > 0 && runs_on(*o, r, type_of[t], ti[t], tk[t]);
    if (!ok) return -6;
  }
  std::vector<std::vector<int64_t>> succ(nt);
  std::vector<int> indeg(nt, 0);
  for (auto& e : E) {
    succ[e.first].push_back(e.second);
    ++indeg[e.second];
  }
  // dmdas priority: bottom level with each type's fastest time over the classes (L655-660)
  double fastest[4];
  for (int t = 0; t < 4; ++t) {
    fastest[t] = INFINITY;
    for (int r = 0; r < R; ++r) {
      const double v = o->time[r][t];
      if (o->workers[r] > 0 && v >= 0.0 && !std::isinf(v)) fastest[t] = std::min(fastest[t], v);
    }
    if (std::isinf(fastest[t])) fastest[t] = 0.0;
  }
  const std::vector<double> prio = bottom_levels(N, fastest);
  // per-worker deques of assigned tasks (StarPU's dm* push tasks to worker queues when ready)
  std::vector<std::vector<int64_t>> wq(W);
  std::vector<double> exp_free(W, 0.0);  // when the worker's queue is expected to drain
  std::vector<char> busy(W, 0);
  std::vector<double> t0(nt, 0.0), t1(nt, 0.0);
  std::vector<int> twork(nt, -1);
  using Ev = std::pair<double, int>;  // (end time, worker): earliest first, then lowest worker
  std::priority_queue<Ev, std::vector<Ev>, std::greater<Ev>> events;
  std::vector<int64_t> running(W, -1);

  if (o->policy == CHOL_SIM_FIXED)
    for (int64_t t = 0; t < nt; ++t) {
      const int w = o->fixed_worker[t];
      if (w < 0 || w >= W || !runs_on(*o, wcls[w], type_of[t], ti[t], tk[t])) return -6;
    }
  auto assign = [&](std::vector<int64_t>& ready, double now) {
    if (o->policy == CHOL_SIM_FIXED) {  // the injected schedule's worker
      for (int64_t t : ready) {
        wq[o->fixed_worker[t]].push_back(t);
        twork[t] = o->fixed_worker[t];
      }
      ready.clear();
      return;
    }
    if (o->policy == 1)  // dmdas: highest priority first (ties: lower id)
      std::stable_sort(ready.begin(), ready.end(), [&](int64_t a, int64_t b) { return prio[a] > prio[b]; });
    for (int64_t t : ready) {
      int best = -1;
      double bend = 0.0;
      for (int w = 0; w < W; ++w) {
        if (!runs_on(*o, wcls[w], type_of[t], ti[t], tk[t])) continue;
        const double end = std::max(exp_free[w], now) + o->time[wcls[w]][type_of[t]];
        if (best < 0 || end < bend) best = w, bend = end;  // minimum completion time (L645-651)
      }
      wq[best].push_back(t);
      exp_free[best] = bend;
      twork[t] = best;
    }
    ready.clear();
  };
  // CHOL_SIM_FIXED: position of each worker in its injected order (next rank to run)
  std::vector<std::vector<int64_t>> worder(W);
  std::vector<size_t> wnext(W, 0);
  if (o->policy == CHOL_SIM_FIXED) {
    for (int64_t t = 0; t < nt; ++t) worder[o->fixed_worker[t]].push_back(t);
    for (auto& v : worder)
      std::stable_sort(v.begin(), v.end(), [&](int64_t a, int64_t b) { return o->fixed_rank[a] < o->fixed_rank[b]; });
  }
  auto start_idle = [&](double now) {
    for (int w = 0; w < W; ++w) {
      if (busy[w] || wq[w].empty()) continue;
      if (o->policy == CHOL_SIM_FIXED) {  // only the worker's next task in the injected order
        if (wnext[w] >= worder[w].size()) continue;
        const int64_t t = worder[w][wnext[w]];
        auto it = std::find(wq[w].begin(), wq[w].end(), t);
        if (it == wq[w].end()) continue;  // not ready yet
        wq[w].erase(it);
        ++wnext[w];
        busy[w] = 1;
        running[w] = t;
        t0[t] = now;
        t1[t] = now + o->time[wcls[w]][type_of[t]];
        events.push(Ev(t1[t], w));
        continue;
      }
      size_t pick = 0;
      if (o->policy == 1)
        for (size_t q = 1; q < wq[w].size(); ++q)
          if (prio[wq[w][q]] > prio[wq[w][pick]]) pick = q;
      const int64_t t = wq[w][pick];
      wq[w].erase(wq[w].begin() + pick);
      busy[w] = 1;
      running[w] = t;
      t0[t] = now;
      t1[t] = now + o->time[wcls[w]][type_of[t]];
      events.push(Ev(t1[t], w));
    }
  };
  std::vector<int64_t> ready;
  for (int64_t t = 0; t < nt; ++t)
    if (indeg[t] == 0) ready.push_back(t);
  assign(ready, 0.0);
  start_idle(0.0);
  double mk = 0.0;
  int64_t done = 0;
  while (!events.empty()) {
    const double now = events.top().first;
    // every completion at this instant, then the released tasks, then idle workers
    while (!events.empty() && events.top().first == now) {
      const int w = events.top().second;
      events.pop();
      const int64_t t = running[w];
      busy[w] = 0;
      running[w] = -1;
      ++done;
      mk = std::max(mk, t1[t]);
      for (int64_t s : succ[t])
        if (--indeg[s] == 0) ready.push_back(s);
    }
    assign(ready, now);
    start_idle(now);
  }
  if (done != nt) return -6;
  *makespan = mk;
  if (recs)
    for (int64_t t = 0; t < nt && t < cap; ++t) {
      chol_task_rec_t& r = recs[t];
      r.type = (uint8_t)type_of[t];
      r.gpu = (uint8_t)wcls[twork[t]];
      r.worker = (uint16_t)twork[t];
      r.i = ti[t];
      r.j = tj[t];
      r.k = tk[t];
      r.t0_ns = (uint64_t)std::llround(t0[t] * 1e9);
      r.t1_ns = (uint64_t)std::llround(t1[t] * 1e9);
    }
  return 0;
}

// ------------------------------------------------------------------ exact schedules (NEXT-4)
namespace {
struct ExactSearch {
  int64_t nt = 0;
  int W = 0, R = 0;
  const chol_sim_opts_t* o = nullptr;
  std::vector<int> type_of, ti, tk, wcls;
  std::vector<std::vector<int>> succ, pred;
  std::vector<int> topo;                 // a topological order (task ids are one)
  std::vector<double> fast, blev;        // fastest time over the allowed classes; bottom level
  std::vector<std::vector<int>> cls_workers;
  // state
  std::vector<double> fin, st;
  std::vector<int> wk, npred;
  std::vector<double> wfree;
  double best = INFINITY;
  std::vector<double> best_st;
  std::vector<int> best_wk;
  int64_t nodes = 0, limit = 0;
  bool stopped = false;
  std::vector<double> es;  // scratch: earliest starts

  double lower_bound(double cur_mk) {
    // longest remaining path: earliest start of every unscheduled task (scheduled
    // predecessors: their finish; unscheduled ones: their earliest start + fastest time)
    double lb = cur_mk, work = 0.0;
    for (int t : topo) {
      if (fin[t] >= 0.0) continue;
      double e = 0.0;
      for (int p : pred[t]) e = std::max(e, fin[p] >= 0.0 ? fin[p] : es[p] + fast[p]);
      es[t] = e;
      lb = std::max(lb, e + blev[t]);
      work += fast[t];
    }
    double busy = 0.0;
    for (int w = 0; w < W; ++w) busy += wfree[w];
    return std::max(lb, (busy + work) / W);
  }

  void dfs(int nsched, double cur_mk, double cursor, int last_task) {
    if (stopped) return;
    if (nsched == nt) {
      if (cur_mk < best) {
        best = cur_mk;
        best_st = st;
        best_wk = wk;
      }
      return;
    }
    if (++nodes > limit) {
      stopped = true;
      return;
    }
    if (lower_bound(cur_mk) >= best - 1e-12) return;
    struct Cand {
      double est, ect;
      int t, w;
    };
    std::vector<Cand> cand;
    for (int t = 0; t < nt; ++t) {
      if (fin[t] >= 0.0 || npred[t] != 0) continue;
      double ready = 0.0;
      for (int p : pred[t]) ready = std::max(ready, fin[p]);
      for (int r = 0; r < R; ++r) {
        if (cls_workers[r].empty() || !runs_on(*o, r, type_of[t], ti[t], tk[t])) continue;
        int bw = cls_workers[r][0];
        for (int w : cls_workers[r])
          if (wfree[w] < wfree[bw]) bw = w;
        const double est = std::max(ready, wfree[bw]);
        // start-time order (ties by task id): every semi-active schedule is generated once
        if (est < cursor - 1e-12 || (est <= cursor + 1e-12 && t <= last_task && nsched > 0)) continue;
        cand.push_back({est, est + o->time[r][type_of[t]], t, bw});
      }
    }
    std::sort(cand.begin(), cand.end(), [](const Cand& a, const Cand& b) {
      return a.ect != b.ect ? a.ect < b.ect : (a.est != b.est ? a.est < b.est : a.t < b.t);
    });
    for (const Cand& c : cand) {
      if (c.ect >= best - 1e-12) continue;
      const double old_free = wfree[c.w];
      fin[c.t] = c.ect;
      st[c.t] = c.est;
      wk[c.t] = c.w;
      wfree[c.w] = c.ect;
      for (int s : succ[c.t]) --npred[s];
      dfs(nsched + 1, std::max(cur_mk, c.ect), c.est, c.t);
      for (int s : succ[c.t]) ++npred[s];
      wfree[c.w] = old_free;
      fin[c.t] = -1.0;
      wk[c.t] = -1;
      if (stopped) return;
    }
  }
};
}  // namespace

extern "C" int chol_optimal_schedule(int64_t N, const chol_sim_opts_t* o, int64_t node_limit, double* makespan,
                                     int* optimal, int32_t* worker, int32_t* rank, int64_t* nodes) {
  if (N <= 0) return -1;
  if (!o || !makespan) return -4;
  if (N > 8 || o->nclasses < 1 || o->nclasses > CHOL_SIM_MAX_CLASSES) return -6;
  ExactSearch S;
  S.o = o;
  S.R = o->nclasses;
  S.cls_workers.resize(S.R);
  for (int r = 0; r < S.R; ++r) {
    if (o->workers[r] < 0) return -6;
    for (int w = 0; w < o->workers[r]; ++w) {
      S.cls_workers[r].push_back((int)S.wcls.size());
      S.wcls.push_back(r);
    }
  }
  S.W = (int)S.wcls.size();
  if (S.W == 0) return -6;
  std::vector<std::pair<int64_t, int64_t>> E;
  build_task_dag(N, E, S.type_of);
  S.nt = n_tasks(N);
  S.ti.assign(S.nt, 0);
  S.tk.assign(S.nt, 0);
  for (int64_t k = 0; k < N; ++k) {
    S.ti[id_potrf(N, k)] = (int)k, S.tk[id_potrf(N, k)] = (int)k;
    for (int64_t i = k + 1; i < N; ++i) S.ti[id_trsm(N, i, k)] = (int)i, S.tk[id_trsm(N, i, k)] = (int)k;
  }
  S.succ.assign(S.nt, {});
  S.pred.assign(S.nt, {});
  for (auto& e : E) {
    S.succ[e.first].push_back((int)e.second);
    S.pred[e.second].push_back((int)e.first);
  }
  // topological order (Kahn)
  std::vector<int> indeg(S.nt, 0);
  for (auto& e : E) ++indeg[e.second];
  for (int t = 0; t < S.nt; ++t)
    if (!indeg[t]) S.topo.push_back(t);
  for (size_t h = 0; h < S.topo.size(); ++h)
    for (int s : S.succ[S.topo[h]])
      if (--indeg[s] == 0) S.topo.push_back(s);
  S.fast.assign(S.nt, INFINITY);
  for (int t = 0; t < S.nt; ++t) {
    for (int r = 0; r < S.R; ++r)
      if (o->workers[r] > 0 && runs_on(*o, r, S.type_of[t], S.ti[t], S.tk[t]))
        S.fast[t] = std::min(S.fast[t], o->time[r][S.type_of[t]]);
    if (std::isinf(S.fast[t])) return -6;
  }
  S.blev.assign(S.nt, 0.0);
  for (int h = (int)S.topo.size() - 1; h >= 0; --h) {
    const int t = S.topo[h];
    double m = 0.0;
    for (int s : S.succ[t]) m = std::max(m, S.blev[s]);
    S.blev[t] = S.fast[t] + m;
  }
  // incumbent: the dmdas replay
  {
    chol_sim_opts_t od = *o;
    od.policy = CHOL_SIM_DMDAS;
    std::vector<chol_task_rec_t> recs(S.nt);
    double mk = 0.0;
    if (chol_simulate(N, &od, &mk, recs.data(), S.nt) == 0) {
      S.best = mk + 1e-9;  // strictly better schedules only; kept if none is found
      S.best_st.resize(S.nt);
      S.best_wk.resize(S.nt);
      for (int t = 0; t < S.nt; ++t) {
        S.best_st[t] = recs[t].t0_ns * 1e-9;
        S.best_wk[t] = recs[t].worker;
      }
    }
  }
  S.fin.assign(S.nt, -1.0);
  S.st.assign(S.nt, 0.0);
  S.wk.assign(S.nt, -1);
  S.npred.assign(S.nt, 0);
  for (int t = 0; t < S.nt; ++t) S.npred[t] = (int)S.pred[t].size();
  S.wfree.assign(S.W, 0.0);
  S.es.assign(S.nt, 0.0);
  S.limit = node_limit > 0 ? node_limit : (int64_t)200000000;
  S.dfs(0, 0.0, 0.0, -1);
  if (S.best_wk.empty()) return -6;
  // the schedule's exact makespan (the dmdas incumbent carried a 1e-9 guard)
  double mk = 0.0;
  for (int t = 0; t < S.nt; ++t) mk = std::max(mk, S.best_st[t] + o->time[S.wcls[S.best_wk[t]]][S.type_of[t]]);
  *makespan = mk;
  if (optimal) *optimal = S.stopped ? 0 : 1;
  if (nodes) *nodes = S.nodes;
  if (worker || rank) {
    std::vector<int> ord(S.nt);
    for (int t = 0; t < S.nt; ++t) ord[t] = t;
    std::stable_sort(ord.begin(), ord.end(), [&](int a, int b) { return S.best_st[a] < S.best_st[b]; });
    for (int r = 0; r < S.nt; ++r) {
      if (worker) worker[ord[r]] = S.best_wk[ord[r]];
      if (rank) rank[ord[r]] = r;
    }
  }
  return 0;
}
