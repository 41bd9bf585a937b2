// solver.cpp -- host share solver (accel_solve / accel_demand_of).
//
// PAPER.md §3 (lines 483-542): per kernel i the work-groups allowed by threads,
// local memory and registers are x_i = T/(K w_i), y_i = L/(K m_i),
// z_i = R/(K r_i); the quota is their minimum; being Diophantine the result
// may be conservative, and a greedy heuristic adds work-groups across the
// kernels until the resources saturate.  B200 readings (DESIGN.md
// R-solver-1..9): floors; CTA slots as a fourth resource; warp/SMSP register
// allocation and reserved/rounded shared memory in the demand vector; a
// per-SM packing check F after the closed form; class-symmetric decrement and
// greedy so identical kernels get identical quotas.  Must agree exactly with
// the oracle (tests/test_solver_parity.py).
#include <algorithm>
#include <cstdint>
#include <vector>

#include "accel.h"

namespace {

struct Caps {
  int64_t sms, thr, regs, smem, ctas;
  static constexpr int64_t kSmsp = 4;
  static constexpr int64_t kRegGran = 256;
  static constexpr int64_t kSmemGran = 128;
  static constexpr int64_t kSmemReserved = 1024;
  static constexpr int64_t kMaxSmemPerCta = 232448;
  static constexpr int64_t kMaxRegsPerThread = 255;
  int64_t regs_per_smsp() const { return regs / kSmsp; }
};

Caps caps_of(const accel_caps* c) {
  Caps k{148, 2048, 65536, 233472, 32};
  if (c) {
    if (c->sms > 0) k.sms = c->sms;
    if (c->thr_per_sm > 0) k.thr = c->thr_per_sm;
    if (c->regs_per_sm > 0) k.regs = c->regs_per_sm;
    if (c->smem_per_sm > 0) k.smem = c->smem_per_sm;
    if (c->ctas_per_sm > 0) k.ctas = c->ctas_per_sm;
  }
  return k;
}

int64_t cdiv(int64_t a, int64_t b) { return (a + b - 1) / b; }

struct Req {
  int64_t thr, regs, smem, cta, g, w;
  int64_t warps() const { return thr / 32; }
  int64_t rpw() const { return regs / warps(); }
  bool same(const Req& o) const {
    return thr == o.thr && regs == o.regs && smem == o.smem && cta == o.cta && g == o.g && w == o.w;
  }
};

bool valid(const Req& r, const Caps& c) {
  if (r.thr <= 0 || r.thr % 32 || r.thr > c.thr || r.cta != 1 || r.w <= 0) return false;
  if (r.regs <= 0 || r.regs % r.warps() || r.rpw() % Caps::kRegGran) return false;
  if (cdiv(r.warps(), Caps::kSmsp) * r.rpw() > c.regs_per_smsp()) return false;
  if (r.smem <= 0 || r.smem > c.smem) return false;
  return true;
}

// a/b < c/d for positive denominators, exact
bool frac_less(__int128 a, __int128 b, __int128 c, __int128 d) { return a * d < c * b; }

// Per-CTA footprint: the largest share of ONE SM's resources, as (num, den).
void footprint(const Req& r, const Caps& c, __int128* num, __int128* den) {
  const __int128 cand[4][2] = {{r.thr, c.thr}, {r.regs, c.regs}, {r.smem, c.smem}, {r.cta, c.ctas}};
  *num = cand[0][0];
  *den = cand[0][1];
  for (int i = 1; i < 4; ++i)
    if (frac_less(*num, *den, cand[i][0], cand[i][1])) {
      *num = cand[i][0];
      *den = cand[i][1];
    }
}

// R-place-1: indices, largest per-CTA footprint first, ties in arrival order.
std::vector<int> placement_order(const std::vector<Req>& rs, const Caps& c) {
  std::vector<int> ord(rs.size());
  for (size_t i = 0; i < rs.size(); ++i) ord[i] = (int)i;
  std::stable_sort(ord.begin(), ord.end(), [&](int a, int b) {
    __int128 na, da, nb, db;
    footprint(rs[a], c, &na, &da);
    footprint(rs[b], c, &nb, &db);
    return frac_less(nb, db, na, da);  // a's footprint > b's
  });
  return ord;
}

// F(n) (R-solver-3): kernels in placement order, each kernel's CTAs dealt
// round-robin over the SMs from a pointer carried over between kernels, a CTA
// going to the next SM where it fits (thread / CTA-slot / shared-memory sums,
// warps packed round-robin from the least-loaded SMSP); dealt in rounds.
bool feasible(const std::vector<Req>& rs, const std::vector<int64_t>& n, const Caps& c) {
  struct Sm {
    int64_t thr = 0, ctas = 0, smem = 0, sp[Caps::kSmsp] = {0, 0, 0, 0};
  };
  std::vector<Sm> sm((size_t)c.sms);
  auto place = [&](const Sm& s, const Req& r, Sm* out) {
    if (s.thr + r.thr > c.thr || s.ctas + r.cta > c.ctas || s.smem + r.smem > c.smem) return false;
    *out = s;
    int start = 0;
    for (int x = 1; x < Caps::kSmsp; ++x)
      if (s.sp[x] < s.sp[start]) start = x;
    const int64_t w = r.warps(), rpw = r.rpw();
    for (int64_t x = 0; x < w; ++x) out->sp[(start + x) % Caps::kSmsp] += rpw;
    for (int x = 0; x < Caps::kSmsp; ++x)
      if (out->sp[x] > c.regs_per_smsp()) return false;
    out->thr += r.thr;
    out->ctas += r.cta;
    out->smem += r.smem;
    return true;
  };
  std::vector<std::pair<int64_t, Sm>> fit;
  fit.reserve((size_t)c.sms);
  int64_t p = 0;
  for (int i : placement_order(rs, c)) {
    const Req& r = rs[(size_t)i];
    int64_t left = n[(size_t)i];
    while (left > 0) {
      fit.clear();
      for (int64_t j = 0; j < c.sms && (int64_t)fit.size() < left; ++j) {
        const int64_t k = (p + j) % c.sms;
        Sm nx;
        if (place(sm[(size_t)k], r, &nx)) fit.emplace_back(k, nx);
      }
      if (fit.empty()) return false;
      for (auto& f : fit) sm[(size_t)f.first] = f.second;
      left -= (int64_t)fit.size();
      p = (fit.back().first + 1) % c.sms;
    }
  }
  return true;
}

// dominant share of a request holding n CTAs: max_r n*d_r/(S*cap_r) as (num, den)
void dominant(const Req& r, int64_t n, const Caps& c, __int128* num, __int128* den) {
  const __int128 cand[4][2] = {{(__int128)n * r.thr, (__int128)c.sms * c.thr},
                               {(__int128)n * r.regs, (__int128)c.sms * c.regs},
                               {(__int128)n * r.smem, (__int128)c.sms * c.smem},
                               {(__int128)n * r.cta, (__int128)c.sms * c.ctas}};
  *num = cand[0][0];
  *den = cand[0][1];
  for (int i = 1; i < 4; ++i)
    if (frac_less(*num, *den, cand[i][0], cand[i][1])) {
      *num = cand[i][0];
      *den = cand[i][1];
    }
}

}  // namespace

extern "C" int accel_placement_order(const accel_caps* caps, const accel_demand* d, int32_t k, int32_t* order_out) {
  if (k < 0 || (k > 0 && (!d || !order_out))) return ACCEL_EINVAL;
  const Caps c = caps_of(caps);
  std::vector<Req> rs((size_t)k);
  for (int32_t i = 0; i < k; ++i)
    rs[(size_t)i] = Req{d[i].thr, d[i].regs, d[i].smem, d[i].cta, d[i].grid_vgs, d[i].weight ? d[i].weight : 1};
  for (const Req& r : rs)
    if (!valid(r, c)) return ACCEL_ENOFIT;
  const std::vector<int> ord = placement_order(rs, c);
  for (int32_t i = 0; i < k; ++i) order_out[i] = ord[(size_t)i];
  return ACCEL_OK;
}

extern "C" int accel_demand_of(const accel_caps* caps, uint32_t block_threads, uint32_t regs_per_thread,
                               uint32_t smem_bytes, uint32_t grid_vgs, uint32_t weight,
                               accel_demand* out) {
  if (!out || block_threads == 0) return ACCEL_EINVAL;
  const Caps c = caps_of(caps);
  const int64_t warps = cdiv(block_threads, 32);
  const int64_t rpw = cdiv(32 * (int64_t)regs_per_thread, Caps::kRegGran) * Caps::kRegGran;
  const int64_t smem = cdiv((int64_t)smem_bytes + Caps::kSmemReserved, Caps::kSmemGran) * Caps::kSmemGran;
  if (32 * warps > c.thr || (int64_t)smem_bytes > Caps::kMaxSmemPerCta ||
      (int64_t)regs_per_thread > Caps::kMaxRegsPerThread ||
      cdiv(warps, Caps::kSmsp) * rpw > c.regs_per_smsp() || smem > c.smem)
    return ACCEL_ENOFIT;
  out->thr = (uint32_t)(32 * warps);
  out->regs = (uint32_t)(rpw * warps);
  out->smem = (uint32_t)smem;
  out->cta = 1;
  out->grid_vgs = grid_vgs;
  out->weight = weight ? weight : 1;
  return ACCEL_OK;
}

extern "C" int accel_solve(const accel_caps* caps, const accel_demand* d, int32_t k, uint32_t* quota_out) {
  if (k < 0 || (k > 0 && (!d || !quota_out))) return ACCEL_EINVAL;
  const Caps c = caps_of(caps);
  std::vector<Req> rs(k);
  for (int i = 0; i < k; ++i) {
    rs[i] = Req{d[i].thr, d[i].regs, d[i].smem, d[i].cta, d[i].grid_vgs, d[i].weight ? d[i].weight : 1};
    if (!valid(rs[i], c)) return ACCEL_ENOFIT;
  }
  // classes of identical requests, in order of first arrival
  std::vector<std::vector<int>> cls;
  for (int i = 0; i < k; ++i) {
    bool placed = false;
    for (auto& m : cls)
      if (rs[m[0]].same(rs[i])) {
        m.push_back(i);
        placed = true;
        break;
      }
    if (!placed) cls.push_back({i});
  }
  // closed form on device totals (weights scale the share)
  int64_t W = 0;
  for (auto& r : rs)
    if (r.g > 0) W += r.w;
  std::vector<int64_t> n(k, 0);
  for (int i = 0; i < k; ++i) {
    const Req& r = rs[i];
    if (r.g == 0) continue;
    const int64_t x = (c.sms * c.thr * r.w) / (W * r.thr);
    const int64_t z = (c.sms * c.regs * r.w) / (W * r.regs);
    const int64_t y = (c.sms * c.smem * r.w) / (W * r.smem);
    const int64_t s = (c.sms * c.ctas * r.w) / (W * r.cta);
    n[i] = std::max<int64_t>(1, std::min({x, y, z, s, r.g}));
  }
  // decrement whole classes with the largest dominant share until F holds
  while (!feasible(rs, n, c)) {
    int best = -1;
    __int128 bn = 0, bd = 1;
    for (size_t ci = 0; ci < cls.size(); ++ci) {
      const int i = cls[ci][0];
      if (n[i] <= 1) continue;
      __int128 num, den;
      dominant(rs[i], n[i], c, &num, &den);
      if (best < 0 || !frac_less(num, den, bn, bd)) {  // >= : later class wins ties
        best = (int)ci;
        bn = num;
        bd = den;
      }
    }
    if (best < 0) break;  // 1 CTA each does not pack (tiny devices only)
    for (int i : cls[best]) n[i] -= 1;
  }
  // class-symmetric greedy fill
  for (;;) {
    bool accepted = false;
    for (auto& m : cls) {
      bool room = true;
      for (int i : m)
        if (n[i] + 1 > rs[i].g) room = false;
      if (!room) continue;
      for (int i : m) n[i] += 1;
      if (feasible(rs, n, c))
        accepted = true;
      else
        for (int i : m) n[i] -= 1;
    }
    if (!accepted) break;
  }
  for (int i = 0; i < k; ++i) quota_out[i] = (uint32_t)n[i];
  return ACCEL_OK;
}
