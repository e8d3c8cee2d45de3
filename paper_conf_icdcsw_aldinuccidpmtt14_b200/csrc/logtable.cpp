// logtable.cpp — host construction of the CWC-log table (reading R4).
//
// For i in [0, 128): the reduced argument z of table index i lies in
// [bits(OFF + i*2^45), bits(OFF + (i+1)*2^45)), OFF = 0x3fe6000000000000 (z in [0.6875, 1.375)).
// c_i is the midpoint of that range; invc_i = 1/c_i (IEEE division), except the two ranges
// touching 1.0 (i = 79, 80) where invc_i = 1 so that r = z - 1 is exact near log's zero;
// log(c_i) = -log(invc_i) is evaluated in x87 extended precision and split into a double-double
// (logc_i, logclo_i).  Every step is a correctly rounded operation or the host libm's logl.
#include <cmath>
#include <cstdint>
#include <cstring>

#include "device/cwc_params.h"

namespace cwc {

void build_log_table(cwc_logtab_entry* tab) {
    const uint64_t OFF = 0x3fe6000000000000ULL;
    for (int i = 0; i < 128; ++i) {
        uint64_t blo = OFF + ((uint64_t)i << 45), bhi = OFF + ((uint64_t)(i + 1) << 45);
        double zlo, zhi;
        std::memcpy(&zlo, &blo, 8);
        std::memcpy(&zhi, &bhi, 8);
        const double mid = (zlo + zhi) / 2.0;
        const double invc = (i == 79 || i == 80) ? 1.0 : 1.0 / mid;
        const long double l = -logl((long double)invc);
        tab[i].invc = invc;
        tab[i].logc = (double)l;
        tab[i].logclo = (double)(l - (long double)tab[i].logc);
    }
}

}  // namespace cwc
