cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag2.log; : > $O
run() { echo "== $*" >> $O; timeout 100 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run DIAG_TIMEOUT=60 DIAG_N=2000 python tools/split_diag.py C5 33 3
run CULI_LIB=scratch/libculi_wd.so DIAG_TIMEOUT=60 DIAG_N=2000 python tools/split_diag.py C5 1 3
run CULI_LIB=scratch/libculi_wd.so DIAG_TIMEOUT=60 DIAG_N=2000 CULI_WAIT_MS=1000 python tools/split_diag.py C5 1 1
run CULI_LIB=scratch/libculi_wd.so DIAG_TIMEOUT=60 DIAG_N=500 python tools/split_diag.py C5 1 5
grep -v "Exception ignored\|Traceback\|culi.py\|NoneType" $O
