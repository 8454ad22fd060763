// inst.cu -- one translation unit per (key width, key kind) instantiates the launch
// sequences of hrs_host.cuh (the build compiles it four times, in parallel):
//   HRS_INST_KB = 4 | 8   key bytes;   HRS_INST_TY = 0 | 1   unsigned / signed-float keys
// (the order-preserving bijection is compiled into the kernels only for TY = 1).
// HRS_ONLY_TYPES=44 or 88: experiment builds instantiate one unsigned key/value pair only.
#include "hrs_host.cuh"

#ifndef HRS_INST_KB
#error "HRS_INST_KB must be 4 or 8"
#endif
#ifndef HRS_INST_TY
#define HRS_INST_TY 0
#endif
#ifndef HRS_ONLY_TYPES
#define HRS_ONLY_TYPES 0
#endif

namespace hrs_host {

#if HRS_INST_KB == 4
using KI = uint32_t;
#else
using KI = unsigned long long;
#endif
constexpr bool TYI = HRS_INST_TY != 0;

static hrs_status sort_inst(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin,
                            void *vout, cudaStream_t st, int dev, int sms, const uint64_t *grouped) {
#if HRS_ONLY_TYPES
    if (TYI || HRS_ONLY_TYPES != 11 * HRS_INST_KB || vb != HRS_INST_KB) return HRS_ERROR_INVALID_VALUE;
    return run_sort<KI, KI, false>(pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
#else
    if (vb == 0) return run_sort<KI, NoVal, TYI>(pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
    if (vb == 4) return run_sort<KI, uint32_t, TYI>(pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
    return run_sort<KI, unsigned long long, TYI>(pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
#endif
}

#if HRS_INST_TY == 0
static hrs_status block_inst(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin,
                             void *vout, uint64_t *h, uint64_t *o, bool sc, cudaStream_t st, int dev, int sms) {
#if HRS_ONLY_TYPES
    (void)vb; (void)pl; (void)temp; (void)kin; (void)kout; (void)vin; (void)vout; (void)h; (void)o; (void)sc;
    (void)st; (void)dev; (void)sms;
    return HRS_ERROR_INVALID_VALUE;
#else
    if (vb == 0) return run_block<KI, NoVal>(pl, temp, kin, kout, vin, vout, h, o, sc, st, dev, sms);
    if (vb == 4) return run_block<KI, uint32_t>(pl, temp, kin, kout, vin, vout, h, o, sc, st, dev, sms);
    return run_block<KI, unsigned long long>(pl, temp, kin, kout, vin, vout, h, o, sc, st, dev, sms);
#endif
}
#endif

#if HRS_INST_KB == 4 && HRS_INST_TY == 0
hrs_status sort_k4(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                   cudaStream_t st, int dev, int sms, const uint64_t *grouped) {
    return sort_inst(vb, pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
}
hrs_status block_k4(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    uint64_t *h, uint64_t *o, bool sc, cudaStream_t st, int dev, int sms) {
    return block_inst(vb, pl, temp, kin, kout, vin, vout, h, o, sc, st, dev, sms);
}
#elif HRS_INST_KB == 8 && HRS_INST_TY == 0
hrs_status sort_k8(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                   cudaStream_t st, int dev, int sms, const uint64_t *grouped) {
    return sort_inst(vb, pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
}
hrs_status block_k8(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    uint64_t *h, uint64_t *o, bool sc, cudaStream_t st, int dev, int sms) {
    return block_inst(vb, pl, temp, kin, kout, vin, vout, h, o, sc, st, dev, sms);
}
#elif HRS_INST_KB == 4
hrs_status sort_k4t(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    cudaStream_t st, int dev, int sms, const uint64_t *grouped) {
    return sort_inst(vb, pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
}
#else
hrs_status sort_k8t(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    cudaStream_t st, int dev, int sms, const uint64_t *grouped) {
    return sort_inst(vb, pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
}
#endif

}  // namespace hrs_host
