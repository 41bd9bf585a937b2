// guided.cpp -- profile-guided sharing ratios (DESIGN.md R-solver-11; SURVEY
// §8(f) f1).  PAPER.md lines 388-393: the sharing ratio of a request can be
// changed "to reflect priorities"; the paper's own policy is the equal ratio.
// Resource-equal shares give equal SLOWDOWNS only if every kernel slows down
// alike when its share shrinks; on B200 an HBM-bound kernel keeps most of its
// speed on a quarter of the SMs while a compute-bound one slows 4x.  Given each
// request's measured share profile -- isolated time at device fractions
// f_0 = 1 > f_1 > ... (scripts/share_profile.py) -- these ratios make the
// predicted slowdowns equal:
//
//   s_i(f)   = T_i(f) / T_i(1), made non-increasing in f, a power law
//              between profile points (linear in log f / log s, so s ~ 1/f
//              and saturation are represented exactly), s_i(f) = s_i(f_min) *
//              f_min / f below the smallest measured fraction, 1 at f >= 1;
//   f_i(S)   = the smallest f in (0, 1] with s_i(f) <= S;
//   S        = the smallest slowdown with sum_i f_i(S) <= 1 (bisection);
//   w_i      = max(1, round(scale * f_i(S) / max_j f_j(S))).
//
// The solver then splits every resource total in proportion to w (R-solver-7).
// Pure host arithmetic; oracle: oracle/guided_ref.py.
#include <algorithm>
#include <cmath>
#include <cstdint>
#include <vector>

#include "accel.h"

namespace {

struct Curve {
  std::vector<double> f, s;   // ascending f, s non-increasing

  // exponent of the power law on segment [f[j-1], f[j]] (<= 0)
  double expo(size_t j) const { return std::log(s[j] / s[j - 1]) / std::log(f[j] / f[j - 1]); }
  double slowdown(double x) const {
    if (x >= 1.0) return 1.0;
    if (x <= f.front()) return s.front() * f.front() / x;
    for (size_t j = 1; j < f.size(); ++j)
      if (x <= f[j]) return s[j - 1] * std::pow(x / f[j - 1], expo(j));
    return 1.0;
  }
  // smallest x in (0, 1] with slowdown(x) <= S (S >= 1)
  double fraction(double S) const {
    if (S >= s.front()) return std::min(1.0, s.front() * f.front() / S);
    for (size_t j = 1; j < f.size(); ++j)
      if (s[j] <= S)   // s[j-1] > S >= s[j]: the crossing is on this segment
        return std::min(f[j], f[j - 1] * std::pow(S / s[j - 1], 1.0 / expo(j)));
    return 1.0;
  }
};

}  // namespace

extern "C" int accel_guided_weights(int32_t k, int32_t nf, const double* fracs, const double* ms, uint32_t scale,
                                    uint32_t* w_out, double* s_pred) {
  if (k <= 0 || nf <= 0 || !fracs || !ms || !w_out || scale == 0) return ACCEL_EINVAL;
  if (fracs[0] != 1.0) return ACCEL_EINVAL;
  for (int32_t j = 1; j < nf; ++j)
    if (!(fracs[j] < fracs[j - 1]) || !(fracs[j] > 0.0)) return ACCEL_EINVAL;
  std::vector<Curve> cv((size_t)k);
  for (int32_t i = 0; i < k; ++i) {
    const double* t = ms + (size_t)i * nf;
    for (int32_t j = 0; j < nf; ++j)
      if (!(t[j] > 0.0) || !std::isfinite(t[j])) return ACCEL_EINVAL;
    Curve& c = cv[(size_t)i];
    // ascending fractions; slowdown relative to the full device, made
    // non-increasing in f (a larger share never predicts a larger slowdown)
    for (int32_t j = nf - 1; j >= 0; --j) {
      c.f.push_back(fracs[j]);
      c.s.push_back(std::max(1.0, t[j] / t[0]));
    }
    for (size_t j = c.s.size() - 1; j-- > 0;) c.s[j] = std::max(c.s[j], c.s[j + 1]);
    c.s.back() = 1.0;
  }
  auto total = [&](double S) {
    double sum = 0.0;
    for (const Curve& c : cv) sum += c.fraction(S);
    return sum;
  };
  double lo = 1.0, hi = 1.0;
  if (total(1.0) > 1.0) {
    hi = 2.0;
    while (total(hi) > 1.0) hi *= 2.0;
    for (int it = 0; it < 200; ++it) {
      const double mid = 0.5 * (lo + hi);
      (total(mid) > 1.0 ? lo : hi) = mid;
    }
  }
  const double S = hi;
  std::vector<double> fr((size_t)k);
  double fmax = 0.0;
  for (int32_t i = 0; i < k; ++i) {
    fr[(size_t)i] = cv[(size_t)i].fraction(S);
    fmax = std::max(fmax, fr[(size_t)i]);
  }
  for (int32_t i = 0; i < k; ++i) {
    const double w = std::round((double)scale * fr[(size_t)i] / fmax);
    w_out[i] = (uint32_t)std::max(1.0, w);
    if (s_pred) s_pred[i] = cv[(size_t)i].slowdown(fr[(size_t)i]);
  }
  return ACCEL_OK;
}
