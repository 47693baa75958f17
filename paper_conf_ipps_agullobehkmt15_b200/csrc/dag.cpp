// Host-side task graph and makespan bounds (A9).
//
// * Tasks: Algorithm 1 in program order, dense ids of taskid.h.
// * Edges: "direct data dependency" (L213-220) -- each task depends on the last
//   writer of every tile it reads or writes, in program order.
// * Bounds (§III), one resource type (GPU, M = ngpus),
//   DESIGN.md readings R9-R12: area = sum_t N_t T_t^thr / M; chain = N T_P^lat +
//   (N-1)(T_T^lat + T_S^lat); mixed = max(area, chain); critical path = longest DAG
//   path with T^lat weights; GEMM peak = (n^3/3) / (M * 2 nb^3 / T_G^thr).
#include "dag.h"

#include <algorithm>
#include <cstdint>
#include <vector>

#include "../../include/chol.h"
#include "taskid.h"

namespace chol {

void build_task_dag(int64_t N, std::vector<std::pair<int64_t, int64_t>>& edges, std::vector<int>& type_of) {
  const int64_t nt = n_tasks(N);
  type_of.assign(nt, 0);
  edges.clear();
  std::vector<int64_t> last_writer((size_t)(N * (N + 1) / 2), -1);
  std::vector<int64_t> preds;
  auto visit = [&](int64_t task, int type, std::initializer_list<int64_t> reads, int64_t write) {
    type_of[task] = type;
    preds.clear();
    auto touch = [&](int64_t tile) {
      const int64_t w = last_writer[tile];
      if (w >= 0 && std::find(preds.begin(), preds.end(), w) == preds.end()) preds.push_back(w);
    };
    for (int64_t t : reads) touch(t);
    touch(write);
    for (int64_t p : preds) edges.emplace_back(p, task);
    last_writer[write] = task;
  };
  for (int64_t k = 0; k < N; ++k) {
    visit(id_potrf(N, k), T_POTRF, {tile_index(k, k)}, tile_index(k, k));
    for (int64_t i = k + 1; i < N; ++i)
      visit(id_trsm(N, i, k), T_TRSM, {tile_index(k, k), tile_index(i, k)}, tile_index(i, k));
    for (int64_t j = k + 1; j < N; ++j) {
      visit(id_syrk(N, j, k), T_SYRK, {tile_index(j, k), tile_index(j, j)}, tile_index(j, j));
      for (int64_t i = j + 1; i < N; ++i)
        visit(id_gemm(N, i, j, k), T_GEMM, {tile_index(i, k), tile_index(j, k), tile_index(i, j)}, tile_index(i, j));
    }
  }
}

// Program order of the task ids (Algorithm 1 order), a topological order.
static std::vector<int64_t> program_order(int64_t N) {
  std::vector<int64_t> ord;
  ord.reserve(n_tasks(N));
  for (int64_t k = 0; k < N; ++k) {
    ord.push_back(id_potrf(N, k));
    for (int64_t i = k + 1; i < N; ++i) ord.push_back(id_trsm(N, i, k));
    for (int64_t j = k + 1; j < N; ++j) {
      ord.push_back(id_syrk(N, j, k));
      for (int64_t i = j + 1; i < N; ++i) ord.push_back(id_gemm(N, i, j, k));
    }
  }
  return ord;
}

std::vector<double> bottom_levels(int64_t N, const double w[4]) {
  std::vector<std::pair<int64_t, int64_t>> E;
  std::vector<int> type_of;
  build_task_dag(N, E, type_of);
  const int64_t nt = n_tasks(N);
  std::vector<std::vector<int64_t>> succ(nt);
  for (auto& e : E) succ[e.first].push_back(e.second);
  std::vector<double> bl(nt, 0.0);
  auto ord = program_order(N);
  for (auto it = ord.rbegin(); it != ord.rend(); ++it) {
    double tail = 0.0;
    for (int64_t s : succ[*it]) tail = std::max(tail, bl[s]);
    bl[*it] = w[type_of[*it]] + tail;
  }
  return bl;
}

// Multi-GPU layout (2D block-cyclic owner-computes): the tiles this
// rank owns get slots 0..nowned-1 in tile-index order; the remote tiles its tasks read
// (final panel tiles L_kk, L_ik) get cache slots in order of first use.
void dist_layout(int64_t N, int p, int q, int rank, std::vector<int>& slot_map, int* nowned, int* ncached) {
  const int64_t ntiles = N * (N + 1) / 2;
  slot_map.assign(ntiles, -1);
  int s = 0;
  for (int64_t i = 0; i < N; ++i)
    for (int64_t j = 0; j <= i; ++j)
      if (tile_owner_h(i, j, p, q) == rank) slot_map[tile_index(i, j)] = s++;
  *nowned = s;
  auto need = [&](int64_t i, int64_t j) {
    const int64_t t = tile_index(i, j);
    if (slot_map[t] < 0) slot_map[t] = s++;
  };
  for (int64_t k = 0; k < N; ++k) {
    for (int64_t i = k + 1; i < N; ++i)
      if (tile_owner_h(i, k, p, q) == rank) need(k, k);  // TRSM_i_k reads L_kk
    for (int64_t j = k + 1; j < N; ++j) {
      if (tile_owner_h(j, j, p, q) == rank) need(j, k);  // SYRK_j_k reads L_jk
      for (int64_t i = j + 1; i < N; ++i)
        if (tile_owner_h(i, j, p, q) == rank) {  // GEMM_i_j_k reads L_ik, L_jk
          need(i, k);
          need(j, k);
        }
    }
  }
  *ncached = s - *nowned;
}

// slot of every tile in its owner's store
void owner_slots(int64_t N, int p, int q, std::vector<int>& out) {
  out.assign(N * (N + 1) / 2, -1);
  std::vector<int> cnt(p * q, 0);
  for (int64_t i = 0; i < N; ++i)
    for (int64_t j = 0; j <= i; ++j) out[tile_index(i, j)] = cnt[tile_owner_h(i, j, p, q)]++;
}

}  // namespace chol

using namespace chol;

extern "C" int chol_dist_layout(int64_t n, int64_t nb, int p, int q, int rank, int* nowned, int* ncached,
                                int32_t* slot_map, int64_t cap) {
  if (n <= 0) return -1;
  if (nb <= 0 || n % nb) return -2;
  if (p < 1 || q < 1 || rank < 0 || rank >= p * q) return -3;
  std::vector<int> sm;
  int no = 0, nc = 0;
  dist_layout(n / nb, p, q, rank, sm, &no, &nc);
  if (nowned) *nowned = no;
  if (ncached) *ncached = nc;
  if (slot_map)
    for (int64_t t = 0; t < (int64_t)sm.size() && t < cap; ++t) slot_map[t] = sm[t];
  return 0;
}

extern "C" int chol_dag(int64_t N, int64_t* ntasks, int64_t* nedges, int64_t* edges, int64_t cap) {
  if (N <= 0) return -1;
  std::vector<std::pair<int64_t, int64_t>> E;
  std::vector<int> type_of;
  build_task_dag(N, E, type_of);
  if (ntasks) *ntasks = n_tasks(N);
  if (nedges) *nedges = (int64_t)E.size();
  if (edges)
    for (int64_t e = 0; e < (int64_t)E.size() && e < cap; ++e) {
      edges[2 * e] = E[e].first;
      edges[2 * e + 1] = E[e].second;
    }
  return 0;
}

extern "C" int chol_task_id(int64_t N, int type, int i, int j, int k, int64_t* id) {
  if (!id || N <= 0 || k < 0 || k >= N) return -6;
  switch (type) {
    case T_POTRF: *id = id_potrf(N, k); return 0;
    case T_TRSM: if (!(i > k && i < N)) return -6; *id = id_trsm(N, i, k); return 0;
    case T_SYRK: if (!(j > k && j < N)) return -6; *id = id_syrk(N, j, k); return 0;
    case T_GEMM: if (!(i > j && j > k && i < N)) return -6; *id = id_gemm(N, i, j, k); return 0;
  }
  return -6;
}

extern "C" int chol_bounds(int64_t n, int64_t nb, int ngpus, const double* T_lat, const double* T_thr,
                           double* out) {
  if (n <= 0) return -1;
  if (nb <= 0 || n % nb) return -2;
  if (ngpus < 1) return -3;
  if (!T_lat || !T_thr || !out) return -4;
  const int64_t N = n / nb;
  const double M = ngpus;
  const double NP = (double)N, NT = (double)n_trsm(N), NG = (double)n_gemm(N);
  const double area = (NP * T_thr[0] + NT * T_thr[1] + NT * T_thr[2] + NG * T_thr[3]) / M;
  const double chain = NP * T_lat[0] + (NP - 1) * (T_lat[1] + T_lat[2]);
  double cp = 0.0;
  if (N <= 256) {
    auto bl = bottom_levels(N, T_lat);
    cp = *std::max_element(bl.begin(), bl.end());
  } else {
    cp = -1.0;  // not computed (DAG too large for the O(tasks) host DP budget)
  }
  const double RG = 2.0 * (double)nb * nb * nb / T_thr[3];
  const double gpk = ((double)n * n * n / 3.0) / (M * RG);
  out[0] = area;
  out[1] = chain;
  out[2] = std::max(area, chain);
  out[3] = cp;
  out[4] = gpk;
  out[5] = std::max(area, cp);
  return 0;
}

// Owner-area bound (ext): under the fixed 2D block-cyclic owner-computes
// placement no schedule beats the busiest rank's own work,
// max_g sum_{tasks owned by g} T_thr(type); the task owner is the owner of the tile it
// overwrites (POTRF_k -> (k,k), TRSM_i_k -> (i,k), SYRK_j_k -> (j,j), GEMM_i_j_k -> (i,j)).
extern "C" int chol_owner_area(int64_t N, int p, int q, const double* T_thr, double* out, double* per_rank) {
  if (N <= 0) return -1;
  if (p < 1 || q < 1) return -3;
  if (!T_thr || !out) return -4;
  std::vector<double> w((size_t)p * q, 0.0);
  for (int64_t k = 0; k < N; ++k) {
    w[tile_owner_h(k, k, p, q)] += T_thr[0];
    for (int64_t i = k + 1; i < N; ++i) w[tile_owner_h(i, k, p, q)] += T_thr[1];
    for (int64_t j = k + 1; j < N; ++j) {
      w[tile_owner_h(j, j, p, q)] += T_thr[2];
      for (int64_t i = j + 1; i < N; ++i) w[tile_owner_h(i, j, p, q)] += T_thr[3];
    }
  }
  *out = *std::max_element(w.begin(), w.end());
  if (per_rank) std::copy(w.begin(), w.end(), per_rank);
  return 0;
}
