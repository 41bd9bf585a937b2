// metrics.cpp -- sharing metrics of PAPER.md §7.4 (lines 877-913).
//   IS_i = T(s)_i / T(a)_i;  U = max IS / min IS  (Ebrahimi et al. [9])
//   STP = sum T(a)/T(s), ANTT = mean T(s)/T(a)   (named at lines 911-913,
//   formulas not printed: DESIGN.md R-metric-2)
//   O = T(c)/T(t): time all kernels co-execute / time at least one executes.
#include <algorithm>
#include <cstdint>
#include <utility>
#include <vector>

#include "accel.h"

extern "C" int accel_metrics(const double* ta, const double* ts, int32_t k, accel_mix_metrics* out) {
  if (!ta || !ts || !out || k <= 0) return ACCEL_EINVAL;
  double mx = 0.0, mn = 0.0, stp = 0.0, antt = 0.0;
  for (int i = 0; i < k; ++i) {
    if (!(ta[i] > 0.0) || !(ts[i] > 0.0)) return ACCEL_EINVAL;
    const double is = ts[i] / ta[i];
    if (i == 0 || is > mx) mx = is;
    if (i == 0 || is < mn) mn = is;
    stp += ta[i] / ts[i];
    antt += is;
  }
  out->unfairness = mx / mn;
  out->stp = stp;
  out->antt = antt / k;
  out->is_max = mx;
  out->is_min = mn;
  return ACCEL_OK;
}

extern "C" int accel_metrics_weighted(const double* ta, const double* ts, const double* w, int32_t k,
                                      double* wunfairness, double* ws_out) {
  if (!ta || !ts || !w || !wunfairness || k <= 0) return ACCEL_EINVAL;
  double wsum = 0.0;
  for (int i = 0; i < k; ++i) {
    if (!(ta[i] > 0.0) || !(ts[i] > 0.0) || !(w[i] > 0.0)) return ACCEL_EINVAL;
    wsum += w[i];
  }
  const double wbar = wsum / k;
  double mx = 0.0, mn = 0.0;
  for (int i = 0; i < k; ++i) {
    const double ws = ts[i] / ta[i] * w[i] / wbar;
    if (ws_out) ws_out[i] = ws;
    if (i == 0 || ws > mx) mx = ws;
    if (i == 0 || ws < mn) mn = ws;
  }
  *wunfairness = mx / mn;
  return ACCEL_OK;
}

extern "C" int accel_overlap(const double* start, const double* end, int32_t k, double* out) {
  if (!start || !end || !out || k <= 0) return ACCEL_EINVAL;
  std::vector<std::pair<double, double>> iv;
  for (int i = 0; i < k; ++i)
    if (end[i] > start[i]) iv.emplace_back(start[i], end[i]);
  if (iv.empty()) {
    *out = 0.0;
    return ACCEL_OK;
  }
  std::sort(iv.begin(), iv.end());
  double tt = 0.0, a = iv[0].first, b = iv[0].second;
  for (size_t i = 1; i < iv.size(); ++i) {
    if (iv[i].first > b) {
      tt += b - a;
      a = iv[i].first;
      b = iv[i].second;
    } else {
      b = std::max(b, iv[i].second);
    }
  }
  tt += b - a;
  if ((int)iv.size() != k) {  // an empty interval never co-executes with the rest
    *out = 0.0;
    return ACCEL_OK;
  }
  double lo = iv[0].first, hi = iv[0].second;
  for (auto& p : iv) {
    lo = std::max(lo, p.first);
    hi = std::min(hi, p.second);
  }
  *out = tt > 0.0 ? std::max(0.0, hi - lo) / tt : 0.0;
  return ACCEL_OK;
}
