# A/B timing of several builds of libtridiag.so on one GPU box, twice, interleaved:
#   LIBS="new= base=ab/libtridiag_base.so" bash tools/ab_bench.sh OUT spec...
# ("name=" with an empty path = the in-tree build; default LIBS compares the
# in-tree build with ab/libtridiag_base.so); one JSON line per point with "lib".
out=$1; shift
LIBS=${LIBS:-"new= base=ab/libtridiag_base.so"}
for r in 1 2; do
  for nl in $LIBS; do
    name=${nl%%=*}; path=${nl#*=}
    TRIDIAG_LIB_AB=$path python tools/quick_bench.py "$@" | sed "s/^{/{\"lib\": \"$name\", /" >> $out
  done
done
