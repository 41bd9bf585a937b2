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
#include <map>
#include <mutex>
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
// The per-SM packing check F (R-solver-6): requests in placement order (largest
// footprint first), each placed in waves -- a wave visits the SMs round-robin
// from the pointer p and puts one CTA on every SM it still fits, the next wave
// starts after the last SM used.  Feasible iff every request's CTAs were placed.
//
// Packer evaluates F incrementally (the solver's greedy fill asks F after
// every +1, which re-simulated the whole device per trial: 1-3 ms per solve,
// the departure -> growth lag of RESOLVE).  It keeps the device state after
// each prefix of the placement order, so a trial re-places only the requests
// from the first changed one on; and a request whose count grows by one
// continues from its own saved state with one more single-CTA wave.  That
// equals re-placing it from scratch: the extra CTA takes the next SM that
// fits after the last one used -- the rest of the last wave's scan, else a
// new wave from the same pointer.  Same results as a fresh F by construction
// (tests/test_solver_parity.py compares with the oracle's plain F).
struct SmState {
  int64_t thr = 0, ctas = 0, smem = 0, sp[Caps::kSmsp] = {0, 0, 0, 0};
};
struct DevState {
  std::vector<SmState> sm;
  int64_t p = 0;
};

bool place_one(const SmState& s, const Req& r, const Caps& c, SmState* out) {
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
}

// place `count` CTAs of r in waves; false if they do not all fit
bool place_request(DevState* d, const Req& r, int64_t count, const Caps& c,
                   std::vector<std::pair<int64_t, SmState>>* fit) {
  if (count <= 0) return true;
  if (r.warps() % Caps::kSmsp == 0) {
    // the same waves over per-SM capacities (integer arithmetic instead of
    // one trial placement per SM and wave); identical result
    // (r's warps are a multiple of the SMSP count: place_one then adds the
    // same registers to every SMSP whatever SMSP it starts at, so "one more
    // fits" is a plain comparison per resource)
    thread_local std::vector<int64_t> got;
    got.assign((size_t)c.sms, 0);
    const int64_t per_sp = (r.warps() / Caps::kSmsp) * r.rpw(), rps = c.regs_per_smsp();
    auto fits = [&](const SmState& s, int64_t g) {
      return s.thr + g * r.thr <= c.thr && s.ctas + g * r.cta <= c.ctas && s.smem + g * r.smem <= c.smem &&
             std::max({s.sp[0], s.sp[1], s.sp[2], s.sp[3]}) + g * per_sp <= rps;
    };
    int64_t left = count;
    bool ok = true;
    while (left > 0) {
      int64_t placed = 0, last = -1;
      for (int64_t j = 0; j < c.sms && placed < left; ++j) {
        const int64_t k = (d->p + j) % c.sms;
        if (fits(d->sm[(size_t)k], got[(size_t)k] + 1)) {
          got[(size_t)k] += 1;
          placed += 1;
          last = k;
        }
      }
      if (placed == 0) {
        ok = false;
        break;
      }
      left -= placed;
      d->p = (last + 1) % c.sms;
    }
    for (int64_t k = 0; k < c.sms; ++k) {
      const int64_t g = got[(size_t)k];
      if (!g) continue;
      SmState& s = d->sm[(size_t)k];
      s.thr += g * r.thr;
      s.ctas += g * r.cta;
      s.smem += g * r.smem;
      for (int x = 0; x < Caps::kSmsp; ++x) s.sp[x] += g * per_sp;
    }
    return ok;
  }
  int64_t left = count;
  while (left > 0) {
    fit->clear();
    for (int64_t j = 0; j < c.sms && (int64_t)fit->size() < left; ++j) {
      const int64_t k = (d->p + j) % c.sms;
      SmState nx;
      if (place_one(d->sm[(size_t)k], r, c, &nx)) fit->emplace_back(k, nx);
    }
    if (fit->empty()) return false;
    for (auto& f : *fit) d->sm[(size_t)f.first] = f.second;
    left -= (int64_t)fit->size();
    d->p = (fit->back().first + 1) % c.sms;
  }
  return true;
}

class Packer {
 public:
  Packer(const std::vector<Req>& rs, const Caps& c) : rs_(rs), c_(c), ord_(placement_order(rs, c)) {
    pos_.resize(rs.size());
    for (size_t j = 0; j < ord_.size(); ++j) pos_[(size_t)ord_[j]] = j;
    pre_.assign(ord_.size() + 1, DevState{});
    pre_[0].sm.assign((size_t)c.sms, SmState{});
    n_.assign(rs.size(), -1);
  }
  // F(m).  The prefix states before the first request (in placement order)
  // whose count changed since the last call are reused; on failure the
  // states up to the failing request stay valid for m.
  bool eval(const std::vector<int64_t>& m) {
    size_t j0 = ord_.size();
    for (size_t i = 0; i < m.size(); ++i)
      if (m[i] != n_[i]) j0 = std::min(j0, pos_[i]);
    n_ = m;
    valid_ = std::min(valid_, j0);
    for (size_t j = valid_; j < ord_.size(); ++j) {
      pre_[j + 1] = pre_[j];
      if (!place_request(&pre_[j + 1], rs_[(size_t)ord_[j]], n_[(size_t)ord_[j]], c_, &fit_)) {
        valid_ = j;
        ok_ = false;
        return false;
      }
      valid_ = j + 1;
    }
    ok_ = true;
    return true;
  }
  // F(n + 1 for every request in `members`), n = the counts of the last
  // successful eval/try_add; on success the trial becomes the accepted state.
  // Requires the accepted state to pack (else F from scratch on a copy).
  bool try_add(const std::vector<int>& members) {
    std::vector<int64_t> m = n_;
    for (int i : members) m[(size_t)i] += 1;
    if (!ok_) {
      if (eval(m)) return true;
      for (int i : members) m[(size_t)i] -= 1;
      n_ = m;        // back to the accepted counts; re-simulate from scratch next time
      valid_ = 0;
      return false;
    }
    // necessary condition first: the device totals (no packing exceeds them)
    {
      __int128 thr = 0, regs = 0, smem = 0, ctas = 0;
      for (size_t i = 0; i < m.size(); ++i) {
        thr += (__int128)m[i] * rs_[i].thr;
        regs += (__int128)m[i] * rs_[i].regs;
        smem += (__int128)m[i] * rs_[i].smem;
        ctas += (__int128)m[i] * rs_[i].cta;
      }
      if (thr > (__int128)c_.sms * c_.thr || regs > (__int128)c_.sms * c_.regs ||
          smem > (__int128)c_.sms * c_.smem || ctas > (__int128)c_.sms * c_.ctas)
        return false;
    }
    size_t j0 = ord_.size();
    for (int i : members) j0 = std::min(j0, pos_[(size_t)i]);
    tmp_.resize(ord_.size() - j0);
    for (size_t j = j0; j < ord_.size(); ++j) {
      const int i = ord_[j];
      DevState& d = tmp_[j - j0];
      bool ok;
      if (j == j0 && m[(size_t)i] == n_[(size_t)i] + 1) {
        d = pre_[j + 1];                    // request i as accepted, plus one CTA
        ok = place_request(&d, rs_[(size_t)i], 1, c_, &fit_);
      } else {
        d = j == j0 ? pre_[j] : tmp_[j - j0 - 1];
        ok = place_request(&d, rs_[(size_t)i], m[(size_t)i], c_, &fit_);
      }
      if (!ok) return false;
    }
    for (size_t j = j0; j < ord_.size(); ++j) std::swap(pre_[j + 1], tmp_[j - j0]);
    n_ = m;
    return true;
  }

 private:
  const std::vector<Req>& rs_;
  const Caps& c_;
  std::vector<int> ord_;
  std::vector<size_t> pos_;
  std::vector<int64_t> n_;
  std::vector<DevState> pre_, tmp_;
  size_t valid_ = 0;   // pre_[0..valid_] hold the states for n_
  bool ok_ = false;    // the last eval packed
  std::vector<std::pair<int64_t, SmState>> fit_;
};

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

namespace {
// Solutions memoised by (device caps, demand vector): the solver is a pure
// function of both, and a serving device sees the same mixes of kernels over
// and over -- a re-solve on a departure then costs a lookup instead of the
// placement search (0.1-1 ms), which is the departure -> growth lag of
// RESOLVE.  Bounded: cleared when it reaches kMemoMax entries.
constexpr size_t kMemoMax = 4096;
std::mutex g_memo_mu;
std::map<std::vector<int64_t>, std::vector<uint32_t>> g_memo;

std::vector<int64_t> memo_key(const Caps& c, const std::vector<Req>& rs) {
  std::vector<int64_t> key = {c.sms, c.thr, c.regs, c.smem, c.ctas};
  for (const Req& r : rs) key.insert(key.end(), {r.thr, r.regs, r.smem, r.cta, r.g, r.w});
  return key;
}
}  // namespace

extern "C" int accel_solve(const accel_caps* caps, const accel_demand* d, int32_t k, uint32_t* quota_out) {
  if (k < 0 || (k > 0 && (!d || !quota_out))) return ACCEL_EINVAL;
  const Caps c = caps_of(caps);
  std::vector<Req> rs(k);
  for (int i = 0; i < k; ++i) {
    rs[i] = Req{d[i].thr, d[i].regs, d[i].smem, d[i].cta, d[i].grid_vgs, d[i].weight ? d[i].weight : 1};
    if (!valid(rs[i], c)) return ACCEL_ENOFIT;
  }
  const std::vector<int64_t> key = memo_key(c, rs);
  {
    std::lock_guard<std::mutex> g(g_memo_mu);
    auto it = g_memo.find(key);
    if (it != g_memo.end()) {
      std::copy(it->second.begin(), it->second.end(), quota_out);
      return ACCEL_OK;
    }
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
  Packer pk(rs, c);
  bool all_work = true;
  for (const Req& r : rs) all_work = all_work && r.g > 0;
  if (cls.size() == 1 && all_work) {
    // One class on an empty device: every SM fills identically (the SMSP
    // register state depends only on the CTA count), so F(n) holds iff
    // members * n <= cap = sms * (CTAs one SM takes) -- the loop below stops
    // at the largest such n (at least 1) in one step instead of one F per CTA
    SmState sm, nx;
    int64_t per_sm = 0;
    while (place_one(sm, rs[0], c, &nx)) {
      sm = nx;
      ++per_sm;
    }
    const int64_t m = (int64_t)cls[0].size(), cap = per_sm * c.sms;
    if (m * n[0] > cap)
      for (int i : cls[0]) n[i] = std::max<int64_t>(1, cap / m);
  }
  while (!pk.eval(n)) {
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
  // class-symmetric greedy fill: every class in turn tries one more CTA per
  // request, rounds until none is accepted
  for (;;) {
    bool accepted = false;
    for (auto& m : cls) {
      bool room = true;
      for (int i : m)
        if (n[i] + 1 > rs[i].g) room = false;
      if (!room) continue;
      if (pk.try_add(m)) {
        for (int i : m) n[i] += 1;
        accepted = true;
      }
    }
    if (!accepted) break;
  }
  for (int i = 0; i < k; ++i) quota_out[i] = (uint32_t)n[i];
  std::lock_guard<std::mutex> g(g_memo_mu);
  if (g_memo.size() >= kMemoMax) g_memo.clear();
  g_memo.emplace(key, std::vector<uint32_t>(quota_out, quota_out + k));
  return ACCEL_OK;
}
